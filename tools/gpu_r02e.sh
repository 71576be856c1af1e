#!/bin/bash
mkdir -p gpurun_out
bash tools/gpu_ab.sh knobs2 "default ow52 cpa6 ow52cpa6 cpa5" "" 2
