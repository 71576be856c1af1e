#!/bin/bash
# 54-column strips (TEA_TB_GEOM 0: overlap 2 x 5 instead of 2 x 6) re-measured on the current
# passes; the 2 x 4 in-process decomposition's kernel-time breakdown
mkdir -p gpurun_out
bash tools/gpu_ab.sh geom "default geom0" "" 2
bash tools/gpu_ab.sh geom_1024 "default geom0" "--n 1024 --no-variants" 1
timeout 600 python bench.py --no-cpu --no-variants --steps 5 --warmup 3 --blocks 2x4 > gpurun_out/blocks_final.log 2>&1
tail -1 gpurun_out/blocks_final.log | python -c "
import json,sys; d=json.loads(sys.stdin.read()); r=d['roofline']
print('2x4', round(d['value'],1), 'it/s', round(d['ms_per_step'],2), 'ms', 'kernel share of step', round(r.get('kernel_time_of_step',0),3), r.get('kernel_ms'), r.get('kernel_avg_us'))"
