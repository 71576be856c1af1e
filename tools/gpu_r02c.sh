#!/bin/bash
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_parity.py -m gpu -q -x -k "fused or overlap or full_size or loop_modes or cppcg1 or kform" > gpurun_out/pytest_tb.log 2>&1; echo "pytest rc=$?"; tail -3 gpurun_out/pytest_tb.log
timeout 600 python -m pytest tests/test_gpu_fullsize.py -m gpu -q -x -s -k 4096 > gpurun_out/fullsize_tb.log 2>&1; echo "fullsize rc=$?"; grep "\^2" gpurun_out/fullsize_tb.log
bash tools/gpu_ab.sh share "default noshare" "" 2
