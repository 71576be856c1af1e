#!/bin/bash
# round 2 final (re-entry, last sources): GPU suite, smoke, the driver bench commands, ncu launch lists + full sets
mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build_final.log 2>&1 || { tail -30 gpurun_out/build_final.log; exit 1; }
timeout 1800 python -m pytest tests -m gpu -q --durations=10 > gpurun_out/pytest_final5.log 2>&1; echo "pytest rc=$?"; tail -3 gpurun_out/pytest_final5.log
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/smoke_final5.log 2>&1; echo "smoke rc=$?"; cat gpurun_out/smoke_final5.log
timeout 1200 python bench.py --impl reference --steps 20 --warmup 5 > gpurun_out/ref_final5.log 2>&1; echo "ref rc=$?"; tail -1 gpurun_out/ref_final5.log | cut -c1-400
timeout 1200 python bench.py --steps 20 --warmup 5 > gpurun_out/bench_final5.log 2>&1; echo "bench rc=$?"; tail -1 gpurun_out/bench_final5.log | cut -c1-400
timeout 600 python bench.py > gpurun_out/bench_default5.log 2>&1; echo "bench default rc=$?"; tail -1 gpurun_out/bench_default5.log | cut -c1-300
bash tools/profile.sh r02g 4096 > gpurun_out/profile_r02g.log 2>&1; echo "profile rc=$?"
ls -la gpurun_out/prof_r02g; du -sh gpurun_out
