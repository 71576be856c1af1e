#!/bin/bash
# 3D SpMV occupancy A/B (TEA_SPMV3_MINB variants from tools/build_variants.py), interleaved (gpurun)
OUT=gpurun_out/spmv3_minb.jsonl; : > $OUT
for rep in 1 2; do
  for v in default s3m4 s3m5 s3m6 s3m8; do
    if [ $v = default ]; then unset TEA_B200_LIB; else export TEA_B200_LIB=build_variants/$v.so; fi
    for m in cg cppcg; do
      timeout 300 python bench.py --no-cpu --n 256 --nz 256 --method $m --steps 5 | tail -1 | sed "s/^{/{\"variant\": \"$v\", /" >> $OUT
    done
  done
done
unset TEA_B200_LIB
python - <<'PY'
import json
for l in open("gpurun_out/spmv3_minb.jsonl"):
    d = json.loads(l); r = d["roofline"]
    print(d["variant"], d["config"]["method"], round(d["value"], 1), "spmv_us",
          round(1e3 * r["kernel_ms"]["spmv"] / 1, 1), r["kernel_gbs"].get("spmv"), d["clocks"]["sm_mhz"])
PY
