#!/bin/bash
# CPPCG1F passes: paired TMEM fetches in the POST pass, 2 CTAs/SM for the PRE pass
mkdir -p gpurun_out
python tools/dump_u.py /tmp/u_new.npz > gpurun_out/dump_ad.log 2>&1
TEA_B200_LIB=build_variants/base.so python tools/dump_u.py /tmp/u_base.npz >> gpurun_out/dump_ad.log 2>&1
python - <<'PY'
import numpy as np
a = np.load("/tmp/u_new.npz"); b = np.load("/tmp/u_base.npz")
for k in a.files:
    print(k, "bitwise" if np.array_equal(a[k], b[k]) else f"DIFF max {np.max(np.abs(a[k]-b[k]))}")
PY
timeout 1500 python -m pytest tests -m gpu -q -x -k "cppcg1f or 4096 or 1024 or fused" > gpurun_out/pytest_ad.log 2>&1; echo "pytest rc=$?"; tail -2 gpurun_out/pytest_ad.log
bash tools/gpu_ab.sh c1f "base default" "" 2
python - <<'PY'
import json
for l in open("gpurun_out/ab_c1f.jsonl"):
    d = json.loads(l); v = d.get("variants", {}).get("cppcg1f", {})
    print(d["variant"], "cppcg1f", round(v.get("value", 0), 1), v.get("kernel_avg_us"))
PY
