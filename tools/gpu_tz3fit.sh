#!/bin/bash
# 3D: wave-fitted plane tiles for the other stencil kernels (TEA_TZ3_FIT variants), interleaved x2 (gpurun)
OUT=gpurun_out/tz3fit.jsonl; : > $OUT
for rep in 1 2; do
  for v in default fit4 fit5 fit8; do
    if [ $v = default ]; then unset TEA_B200_LIB; else export TEA_B200_LIB=build_variants/$v.so; fi
    for m in cppcg cheby; do
      timeout 300 python bench.py --no-cpu --n 256 --nz 256 --method $m --steps 5 | tail -1 | sed "s/^{/{\"variant\": \"$v\", /" >> $OUT
    done
  done
done
unset TEA_B200_LIB
python - <<'PY'
import json
for l in open("gpurun_out/tz3fit.jsonl"):
    d = json.loads(l); r = d["roofline"]
    print(d["variant"], d["config"]["method"], round(d["value"], 1), r["kernel_gbs"], d["clocks"]["sm_mhz"])
PY
