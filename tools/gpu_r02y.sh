#!/bin/bash
# fill-phase skip in the fused passes: bitwise vs TEA_TB_FILL=0, GPU suite, A/B on the headline,
# the 2x4 in-process decomposition and 1024^2
mkdir -p gpurun_out
python tools/dump_u.py gpurun_out/u_fill1.npz > gpurun_out/dump.log 2>&1
TEA_B200_LIB=build_variants/fill0.so python tools/dump_u.py gpurun_out/u_fill0.npz >> gpurun_out/dump.log 2>&1
python - <<'PY'
import numpy as np
a = np.load("gpurun_out/u_fill1.npz"); b = np.load("gpurun_out/u_fill0.npz")
for k in a.files:
    print(k, "bitwise" if np.array_equal(a[k], b[k]) else f"DIFF max {np.max(np.abs(a[k]-b[k]))}")
PY
tail -2 gpurun_out/dump.log
timeout 1500 python -m pytest tests -m gpu -q -x > gpurun_out/pytest_y.log 2>&1; echo "pytest rc=$?"; tail -2 gpurun_out/pytest_y.log
bash tools/gpu_ab.sh fill "fill0 default" "" 2
bash tools/gpu_ab.sh fill_blocks "fill0 default" "--blocks 2x4 --no-variants" 1
bash tools/gpu_ab.sh fill_1024 "fill0 default" "--n 1024 --no-variants" 2
python - <<'PY'
import json
for l in open("gpurun_out/ab_fill.jsonl"):
    d = json.loads(l); v = d.get("variants", {}).get("cppcg1f", {})
    print(d["variant"], "cppcg1f", round(v.get("value", 0), 1), v.get("kernel_avg_us"))
PY
