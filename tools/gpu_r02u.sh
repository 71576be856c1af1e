#!/bin/bash
mkdir -p gpurun_out
timeout 1200 python -m pytest tests/test_gpu_parity.py -m gpu -q -x -k "multiblock or overlap or extended or blocks or stationary or bjcg or kform or cg1" > gpurun_out/pytest_xc.log 2>&1; echo "pytest rc=$?"; tail -2 gpurun_out/pytest_xc.log
timeout 900 python -m pytest tests/test_gpu_fullsize.py -m gpu -q -x -s -k "4096" > gpurun_out/fs.log 2>&1; echo "fs rc=$?"; grep "(2, 4)" gpurun_out/fs.log
OUT=gpurun_out/blocks9.jsonl; : > $OUT
for args in "--blocks 2x4" "--method cg --blocks 2x4" "--method cppcg1f --blocks 2x4" ""; do
  timeout 900 python bench.py --no-cpu --no-variants --steps 5 --warmup 3 $args | tail -1 | sed "s/^{/{\"args\": \"$args\", /" >> $OUT
done
python - <<'PY'
import json
for l in open("gpurun_out/blocks9.jsonl"):
    d = json.loads(l); r = d.get("roofline") or {}
    print(d["args"], round(d["value"], 1), "it/s", round(d["ms_per_step"], 2), "ms", "traced", round(r.get("kernel_time_of_step", 0), 3), {k: round(v,1) for k, v in (r.get("kernel_avg_us") or {}).items()}, "sm", d["clocks"]["sm_mhz"])
PY
