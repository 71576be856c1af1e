#!/bin/bash
mkdir -p gpurun_out
OUT=gpurun_out/blocks5.jsonl; : > $OUT
for args in "--blocks 2x4" "--blocks 2x4 --tile-rows 16" "--blocks 2x4 --tile-rows 32" "--blocks 2x4 --tile-rows 64" "--n 16384 --steps 1" "--n 2048" "--method cg --blocks 2x4" "--method cg --blocks 2x4 --tile-rows 32"; do
  timeout 900 python bench.py --no-cpu --steps 5 --warmup 3 $args | tail -1 | sed "s/^{/{\"args\": \"$args\", /" >> $OUT
done
python - <<'PY'
import json
for l in open("gpurun_out/blocks5.jsonl"):
    d = json.loads(l); r = d.get("roofline") or {}
    print(d["args"], round(d["value"], 1), "it/s", round(d["ms_per_step"], 2), "ms", {k: round(v,1) for k, v in (r.get("kernel_avg_us") or {}).items()}, "sm", d["clocks"]["sm_mhz"])
PY
