#!/bin/bash
# busiest-SM tile model: fused-pass parity subset, then the plans it picks on the bench shapes
mkdir -p gpurun_out
timeout 1500 python -m pytest tests/test_gpu_parity.py tests/test_gpu_fullsize.py -m gpu -q -x -k "fused or tile or cppcg or multiblock or 4096 or 1024" > gpurun_out/pytest_ab.log 2>&1; echo "pytest rc=$?"; tail -2 gpurun_out/pytest_ab.log
OUT=gpurun_out/model_check.jsonl; : > $OUT
run() { timeout 900 python bench.py --no-cpu --no-variants --steps 5 --warmup 3 $1 | tail -1 | sed "s/^{/{\"args\": \"$1\", /" >> $OUT; }
for a in "--n 1024" "--n 2048" "--blocks 2x4" "" "--n 640" "--n 640 --tb-rows 16"; do run "$a"; done
python - <<'PY'
import json
for l in open("gpurun_out/model_check.jsonl"):
    d = json.loads(l); r = d.get("roofline") or {}
    print(d["args"], round(d["value"], 1), "it/s", round(d["ms_per_step"], 2), "ms", {k: round(v,1) for k, v in (r.get("kernel_avg_us") or {}).items()}, "sm", d["clocks"]["sm_mhz"])
PY
