#!/bin/bash
# TEA_NCCL_SELF: the multi-process NCCL code path on one GPU (1-rank communicator)
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_nccl_self.py -m gpu -q -x > gpurun_out/pytest_nccl_self.log 2>&1; echo "pytest rc=$?"; tail -15 gpurun_out/pytest_nccl_self.log
NCCL_DEBUG=WARN timeout 600 python tools/nccl_self_while.py > gpurun_out/nccl_self_while.log 2>&1; echo "while rc=$?"; cat gpurun_out/nccl_self_while.log | tail -12
