#!/bin/bash
# tile-height model candidates (forced --tb-rows) vs the current auto plan
mkdir -p gpurun_out
OUT=gpurun_out/tbrows_model.jsonl; : > $OUT
run() { timeout 900 python bench.py --no-cpu --no-variants $1 | tail -1 | sed "s/^{/{\"args\": \"$1\", /" >> $OUT; }
for rep in 1 2; do
  for r in 0 18 16; do run "--n 1024 --steps 5 --warmup 3 --tb-rows $r"; done
  for r in 0 71 60; do run "--n 2048 --steps 5 --warmup 3 --tb-rows $r"; done
done
for r in 0 382; do run "--n 16384 --steps 1 --warmup 3 --tb-rows $r"; done
python - <<'PY'
import json
for l in open("gpurun_out/tbrows_model.jsonl"):
    d = json.loads(l); r = d.get("roofline") or {}
    print(d["args"], round(d["value"], 1), "it/s", round(d["ms_per_step"], 2), "ms", {k: round(v,1) for k, v in (r.get("kernel_avg_us") or {}).items()}, "sm", d["clocks"]["sm_mhz"])
PY
