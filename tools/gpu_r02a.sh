#!/bin/bash
# round 2, first GPU pass: full-size parity (printed errors), GPU suite, smoke, bench, probes
mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build.log 2>&1 || { tail -30 gpurun_out/build.log; exit 1; }
timeout 1200 python -m pytest tests/test_gpu_fullsize.py -m gpu -x -q -s --durations=10 > gpurun_out/fullsize.log 2>&1; echo "fullsize rc=$?"
timeout 1200 python -m pytest tests -m gpu -x -q --deselect tests/test_gpu_fullsize.py --durations=15 > gpurun_out/pytest_gpu.log 2>&1; echo "pytest rc=$?"
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/smoke.log 2>&1; echo "smoke rc=$?"
timeout 900 python bench.py --steps 20 --warmup 5 > gpurun_out/bench.log 2>&1; echo "bench rc=$?"
timeout 600 python bench.py --steps 20 --warmup 5 --no-trace --no-cpu > gpurun_out/bench_notrace.log 2>&1; echo "bench_notrace rc=$?"
timeout 600 python tools/probe_r02.py > gpurun_out/probe.log 2>&1; echo "probe rc=$?"
tail -3 gpurun_out/fullsize.log gpurun_out/pytest_gpu.log gpurun_out/smoke.log
