#!/bin/bash
# fused-pass tile heights on small blocks after the fill skip (in-graph kernel averages)
mkdir -p gpurun_out
OUT=gpurun_out/tbrows_small.jsonl; : > $OUT
for rows in 0 20 24 28 32; do
  for args in "--blocks 2x4" "--n 1024" "--n 2048"; do
    timeout 600 python bench.py --no-cpu --no-variants --steps 5 --warmup 3 --tb-rows $rows $args | tail -1 | sed "s/^{/{\"args\": \"$args rows=$rows\", /" >> $OUT
  done
done
python - <<'PY'
import json
for l in open("gpurun_out/tbrows_small.jsonl"):
    d = json.loads(l); r = d.get("roofline") or {}
    print(d["args"], round(d["value"], 1), "it/s", round(d["ms_per_step"], 2), "ms", {k: round(v,1) for k, v in (r.get("kernel_avg_us") or {}).items()}, "sm", d["clocks"]["sm_mhz"])
PY
