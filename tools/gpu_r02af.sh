#!/bin/bash
# cp.async staging depth of the fused passes (first P / later P): default 6/2 vs 6/5, 5/5, 5/2
mkdir -p gpurun_out
bash tools/gpu_ab.sh cpa "default cpaL5 cpa5L5 cpa5L2" "" 2
bash tools/gpu_ab.sh cpa_1024 "default cpaL5 cpa5L5 cpa5L2" "--n 1024 --no-variants" 1
python - <<'PY'
import json
for l in open("gpurun_out/ab_cpa.jsonl"):
    d = json.loads(l); v = d.get("variants", {}).get("cppcg1f", {})
    print(d["variant"], "cppcg1f", round(v.get("value", 0), 1), v.get("kernel_avg_us"))
PY
