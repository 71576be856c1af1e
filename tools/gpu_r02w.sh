#!/bin/bash
# scaled recurrence in the fused passes: GPU suite on the in-tree (TEA_TB_SCL=1) build, then an
# interleaved A/B of SCL 0 / 1 / 2 on the headline bench (CPPCG + CPPCG1F variant line)
mkdir -p gpurun_out
timeout 1500 python -m pytest tests -m gpu -q -x > gpurun_out/pytest_w.log 2>&1; echo "pytest rc=$?"; tail -3 gpurun_out/pytest_w.log
bash tools/gpu_ab.sh scl "scl0 default scl2" "" 2
python - <<'PY'
import json
for l in open("gpurun_out/ab_scl.jsonl"):
    d = json.loads(l); v = d.get("variants", {}).get("cppcg1f", {})
    print(d["variant"], "cppcg1f", round(v.get("value", 0), 1), v.get("kernel_avg_us"))
PY
