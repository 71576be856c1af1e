#!/bin/bash
mkdir -p gpurun_out
timeout 600 python -m pytest tests/test_gpu_parity.py -m gpu -q -x -k "fused or overlap or loop_modes or kform" > gpurun_out/pytest_tb.log 2>&1; echo "pytest rc=$?"; tail -2 gpurun_out/pytest_tb.log
for v in geom2; do TEA_B200_LIB=build_variants/$v.so timeout 600 python -m pytest tests/test_gpu_parity.py -m gpu -q -x -k "fused or overlap" > gpurun_out/pytest_$v.log 2>&1; echo "pytest $v rc=$?"; tail -1 gpurun_out/pytest_$v.log; done
bash tools/gpu_ab.sh knobs3 "default geom2 cpa4" "" 2
