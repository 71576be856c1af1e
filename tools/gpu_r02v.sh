#!/bin/bash
# round 2 re-entry: verify HEAD on a fresh box (GPU suite, smoke, driver bench command)
mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build_v.log 2>&1 || { tail -30 gpurun_out/build_v.log; exit 1; }
timeout 1800 python -m pytest tests -m gpu -q --durations=15 > gpurun_out/pytest_v.log 2>&1; echo "pytest rc=$?"; tail -3 gpurun_out/pytest_v.log
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/smoke_v.log 2>&1; echo "smoke rc=$?"; cat gpurun_out/smoke_v.log
timeout 1200 python bench.py --steps 20 --warmup 5 > gpurun_out/bench_v.log 2>&1; echo "bench rc=$?"; tail -1 gpurun_out/bench_v.log | cut -c1-1500
