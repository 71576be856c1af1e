#!/bin/bash
# fused passes at 4 CTAs/SM (128-register cap, spills) vs the default 3
mkdir -p gpurun_out
bash tools/gpu_ab.sh minb4 "default minb4" "" 2
