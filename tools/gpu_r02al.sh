#!/bin/bash
# 4096^2 fused-pass tile heights around the plan (187 rows: one wave at 3 CTAs/SM; 293: 2 per SM)
mkdir -p gpurun_out
OUT=gpurun_out/tbrows_4096.jsonl; : > $OUT
for rep in 1 2; do
  for r in 0 293 250 220 160; do
    timeout 600 python bench.py --no-cpu --no-variants --steps 5 --warmup 3 --tb-rows $r | tail -1 | sed "s/^{/{\"args\": \"rows=$r\", /" >> $OUT
  done
done
python - <<'PY'
import json
for l in open("gpurun_out/tbrows_4096.jsonl"):
    d = json.loads(l); r = d.get("roofline") or {}
    print(d["args"], round(d["value"], 1), {k: round(v, 1) for k, v in (r.get("kernel_avg_us") or {}).items() if k.startswith("tb")}, d["clocks"]["sm_mhz"])
PY
