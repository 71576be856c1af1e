#!/bin/bash
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_parity.py -m gpu -q -x -k "fused or overlap or loop_modes or kform or cppcg or full_size" > gpurun_out/pytest_tb.log 2>&1; echo "pytest tb rc=$?"; tail -3 gpurun_out/pytest_tb.log
bash tools/gpu_ab.sh r6 "default ring8 nopst" "" 2
bash tools/gpu_ab.sh r6f "default ring8" "--method cppcg1f" 1
