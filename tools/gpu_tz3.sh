#!/bin/bash
# 3D plane-tile sweep (--tile-rows = tz of plan_stencil3), 256^3 CG, interleaved x2 (gpurun)
OUT=gpurun_out/tz3.jsonl; : > $OUT
for rep in 1 2; do for tz in 0 16 48 64 128; do
  timeout 300 python bench.py --no-cpu --n 256 --nz 256 --method cg --steps 5 --tile-rows $tz | tail -1 | sed "s/^{/{\"tz\": $tz, /" >> $OUT
done; done
python - <<'PY'
import json
for l in open("gpurun_out/tz3.jsonl"):
    d = json.loads(l); r = d["roofline"]
    print(d["tz"], round(d["value"], 1), r["kernel_gbs"], d["clocks"]["sm_mhz"])
PY
