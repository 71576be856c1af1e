#!/bin/bash
# round 2 GPU pass b: full-size parity, GPU suite, then the ncu launch lists + full sets
mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build.log 2>&1 || { tail -30 gpurun_out/build.log; exit 1; }
timeout 1200 python -m pytest tests/test_gpu_fullsize.py -m gpu -q -s --durations=10 > gpurun_out/fullsize.log 2>&1; echo "fullsize rc=$?"
timeout 1200 python -m pytest tests -m gpu -q --deselect tests/test_gpu_fullsize.py --durations=15 > gpurun_out/pytest_gpu.log 2>&1; echo "pytest rc=$?"
bash tools/profile.sh r02a 4096 > gpurun_out/profile.log 2>&1; echo "profile rc=$?"
tail -3 gpurun_out/fullsize.log; tail -3 gpurun_out/pytest_gpu.log
