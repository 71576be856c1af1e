#!/bin/bash
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_parity.py -m gpu -q -x -k "multiblock or overlap or extended or blocks or fused or tile or cppcg1f" > gpurun_out/pytest_mb.log 2>&1; echo "pytest rc=$?"; tail -2 gpurun_out/pytest_mb.log
OUT=gpurun_out/blocks4.jsonl; : > $OUT
for args in "--blocks 2x4" "--blocks 2x4 --tb-rows 32" "" "--n 1024" "--n 1024 --tb-rows 12" "--method cppcg1f --blocks 2x4" "--method cppcg1f" "--n 16384 --steps 1" "--n 16384 --steps 1 --blocks 2x4"; do
  timeout 900 python bench.py --no-cpu --steps 5 --warmup 3 $args | tail -1 | sed "s/^{/{\"args\": \"$args\", /" >> $OUT
done
python - <<'PY'
import json
for l in open("gpurun_out/blocks4.jsonl"):
    d = json.loads(l); r = d.get("roofline") or {}
    print(d["args"], round(d["value"], 1), "it/s", round(d["ms_per_step"], 2), "ms", {k: round(v,1) for k, v in (r.get("kernel_avg_us") or {}).items()}, "sm", d["clocks"]["sm_mhz"])
PY
