#!/bin/bash
mkdir -p gpurun_out
timeout 600 python -m pytest tests/test_gpu_parity.py -m gpu -q -x -k "fused or overlap or loop_modes" > gpurun_out/pytest_tb.log 2>&1; echo "pytest rc=$?"; tail -2 gpurun_out/pytest_tb.log
bash tools/gpu_ab.sh knobs "default cpaL3 cpaL4 cpa6 spmv5" "" 2
