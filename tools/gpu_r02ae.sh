#!/bin/bash
# SASS-level stall attribution of the fused passes (one full-set capture per pass kind)
mkdir -p gpurun_out
timeout 900 ncu --set full --clock-control none --import-source on -k regex:"k_cheb_tb" -s 2 -c 2 \
   -o gpurun_out/src_tb python tools/kernel_sweep.py --n 4096 --once --iters 40 > gpurun_out/src_tb.log 2>&1
echo "ncu rc=$?"; ls -la gpurun_out/src_tb*
