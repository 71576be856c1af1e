#!/bin/bash
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_parity.py -m gpu -q -x -k "multiblock or overlap or fused" > gpurun_out/pytest_sp.log 2>&1; echo "pytest rc=$?"; tail -2 gpurun_out/pytest_sp.log
OUT=gpurun_out/blocks8.jsonl; : > $OUT
for args in "--blocks 2x4" "--method cg --blocks 2x4" "" "--n 2048" "--method cg"; do
  timeout 900 python bench.py --no-cpu --no-variants --steps 5 --warmup 3 $args | tail -1 | sed "s/^{/{\"args\": \"$args\", /" >> $OUT
done
python - <<'PY'
import json
for l in open("gpurun_out/blocks8.jsonl"):
    d = json.loads(l); r = d.get("roofline") or {}
    print(d["args"], round(d["value"], 1), "it/s", round(d["ms_per_step"], 2), "ms", {k: round(v,1) for k, v in (r.get("kernel_avg_us") or {}).items()}, "sm", d["clocks"]["sm_mhz"])
PY
