#!/bin/bash
# k_bj occupancy A/B (TEA_BJ_MINB), block-Jacobi PCG 4096^2, interleaved x2 (gpurun)
OUT=gpurun_out/bj_minb.jsonl; : > $OUT
for rep in 1 2; do
  for v in default bj8; do
    if [ $v = default ]; then unset TEA_B200_LIB; else export TEA_B200_LIB=build_variants/$v.so; fi
    timeout 300 python bench.py --no-cpu --steps 3 --method bjcg | tail -1 | sed "s/^{/{\"variant\": \"$v\", /" >> $OUT
  done
done
unset TEA_B200_LIB
python - <<'PY'
import json
for l in open("gpurun_out/bj_minb.jsonl"):
    d = json.loads(l); r = d["roofline"]
    print(d["variant"], round(d["value"], 1), r["kernel_gbs"], d["clocks"]["sm_mhz"])
PY
