#!/bin/bash
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_parity.py -m gpu -q -x -k "cppcg1f" > gpurun_out/pytest_1f.log 2>&1; echo "pytest rc=$?"; tail -2 gpurun_out/pytest_1f.log
timeout 900 python -m pytest tests/test_gpu_fullsize.py -m gpu -q -x -s -k "4096 and 7" > gpurun_out/fs.log 2>&1; echo "fs rc=$?"; grep "\^2" gpurun_out/fs.log
OUT=gpurun_out/blocks7.jsonl; : > $OUT
for args in "--method cppcg1f" "" "--method cppcg1f --blocks 2x4" "--blocks 2x4" "--method cppcg1f" ""; do
  timeout 900 python bench.py --no-cpu --steps 5 --warmup 3 $args | tail -1 | sed "s/^{/{\"args\": \"$args\", /" >> $OUT
done
python - <<'PY'
import json
for l in open("gpurun_out/blocks7.jsonl"):
    d = json.loads(l); r = d.get("roofline") or {}
    print(d["args"], round(d["value"], 1), "it/s", round(d["ms_per_step"], 2), "ms", round(d["iterations_per_step"],1), {k: round(v,1) for k, v in (r.get("kernel_avg_us") or {}).items()}, "sm", d["clocks"]["sm_mhz"])
PY
