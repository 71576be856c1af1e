#!/bin/bash
# paired TMEM slot fetches (TEA_TB_LDPAIR) at 3 and 2 CTAs/SM vs the default
mkdir -p gpurun_out
bash tools/gpu_ab.sh pair "default pair3 pair2" "" 2
bash tools/gpu_ab.sh pair_1024 "default pair3 pair2" "--n 1024 --no-variants" 1
