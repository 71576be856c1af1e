#!/bin/bash
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_parity.py -m gpu -q -x -k "fused or cppcg1f or overlap or kform" > gpurun_out/pytest_tb.log 2>&1; echo "pytest rc=$?"; tail -2 gpurun_out/pytest_tb.log
bash tools/gpu_ab.sh stx "default stx0" "" 2
bash tools/gpu_ab.sh stxf "default stx0" "--method cppcg1f" 1
