#!/bin/bash
# round 2 final pass A: GPU suite, smoke, ncu launch lists (cold + warm L2) and full sets
mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build.log 2>&1 || { tail -30 gpurun_out/build.log; exit 1; }
timeout 1800 python -m pytest tests -m gpu -q -s --durations=15 > gpurun_out/pytest_final.log 2>&1; echo "pytest rc=$?"; tail -3 gpurun_out/pytest_final.log
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/smoke_final.log 2>&1; echo "smoke rc=$?"; cat gpurun_out/smoke_final.log
bash tools/profile.sh r02b 4096 > gpurun_out/profile_r02b.log 2>&1; echo "profile rc=$?"
ls -la gpurun_out/prof_r02b
