#!/bin/bash
mkdir -p gpurun_out
timeout 1500 python -m pytest tests -m gpu -q --durations=10 > gpurun_out/pytest_all.log 2>&1; echo "pytest rc=$?"; tail -4 gpurun_out/pytest_all.log
OUT=gpurun_out/blocks.jsonl; : > $OUT
for args in "" "--blocks 2x4" "--method cppcg1f" "--method cppcg1f --blocks 2x4" "--method cppcg1 --blocks 2x4" "--method cg" "--method cg --blocks 2x4"; do
  timeout 600 python bench.py --no-cpu --steps 5 --warmup 3 $args | tail -1 >> $OUT
done
python - <<'PY'
import json
for l in open("gpurun_out/blocks.jsonl"):
    d = json.loads(l); r = d.get("roofline") or {}
    print(d["config"]["method"], d["config"]["parallelism"], round(d["value"], 1), "it/s", round(d["ms_per_step"], 2), "ms", round(d["iterations_per_step"],1), "its", {k: round(v,1) for k, v in (r.get("kernel_ms") or {}).items()}, "sm", d["clocks"]["sm_mhz"])
PY
