#!/bin/bash
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_parity.py -m gpu -q -x -k "overlap or multiblock or stationary or bjcg" > gpurun_out/pytest_ov.log 2>&1; echo "pytest rc=$?"; tail -3 gpurun_out/pytest_ov.log
