#!/bin/bash
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_parity.py -m gpu -q -x -k "cppcg1f" > gpurun_out/pytest_1f.log 2>&1; echo "pytest 1f rc=$?"; tail -15 gpurun_out/pytest_1f.log
timeout 900 python -m pytest tests/test_gpu_parity.py -m gpu -q -k "fused or overlap or loop_modes or kform or cppcg or full_size" > gpurun_out/pytest_tb.log 2>&1; echo "pytest tb rc=$?"; tail -3 gpurun_out/pytest_tb.log
bash tools/gpu_ab.sh m1f "default minb2" "--method cppcg1f" 1
bash tools/gpu_ab.sh m1 "default minb2" "--method cppcg" 1
