#!/bin/bash
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_parity.py -m gpu -q -x -k "fused or overlap or loop_modes or kform or cppcg or full_size or multiblock or conservation" > gpurun_out/pytest_upd.log 2>&1; echo "pytest rc=$?"; tail -2 gpurun_out/pytest_upd.log
timeout 900 python -m pytest tests/test_gpu_fullsize.py -m gpu -q -x -s -k "4096" > gpurun_out/fs.log 2>&1; echo "fs rc=$?"; grep "\^2" gpurun_out/fs.log
bash tools/gpu_ab.sh upd "default noupd" "" 2
bash tools/gpu_ab.sh updb "default noupd" "--blocks 2x4" 1
