#!/bin/bash
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_parity.py -m gpu -q -x -k "multiblock or overlap or extended or blocks" > gpurun_out/pytest_mb.log 2>&1; echo "pytest rc=$?"; tail -3 gpurun_out/pytest_mb.log
timeout 900 python -m pytest tests/test_gpu_fullsize.py -m gpu -q -x -s -k "4096" > gpurun_out/fs.log 2>&1; echo "fs rc=$?"; grep "\^2" gpurun_out/fs.log
OUT=gpurun_out/blocks2.jsonl; : > $OUT
for args in "--blocks 2x4" "--blocks 2x4 --tb-rows 32" "--blocks 2x4 --tb-rows 48" "--blocks 2x4 --tb-rows 64" "--blocks 2x4 --tb-rows 96" "--blocks 2x4 --overlap 1"; do
  timeout 600 python bench.py --no-cpu --steps 5 --warmup 3 $args | tail -1 | sed "s/^{/{\"args\": \"$args\", /" >> $OUT
done
python - <<'PY'
import json
for l in open("gpurun_out/blocks2.jsonl"):
    d = json.loads(l); r = d.get("roofline") or {}
    print(d["args"], round(d["value"], 1), "it/s", round(d["ms_per_step"], 2), "ms", {k: round(v,1) for k, v in (r.get("kernel_ms") or {}).items()}, "sm", d["clocks"]["sm_mhz"])
PY
