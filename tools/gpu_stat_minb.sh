#!/bin/bash
# stand-alone Jacobi / Chebyshev (k_stat) occupancy A/B: TEA_STAT_MINB variants, interleaved x2 (gpurun)
OUT=gpurun_out/stat_minb.jsonl; : > $OUT
for rep in 1 2; do
  for v in default st5 st6 st8; do
    if [ $v = default ]; then unset TEA_B200_LIB; else export TEA_B200_LIB=build_variants/$v.so; fi
    for args in "--method jacobi" "--method cheby" "--n 256 --nz 256 --method jacobi"; do
      timeout 300 python bench.py --no-cpu --steps 3 $args | tail -1 | sed "s/^{/{\"variant\": \"$v\", /" >> $OUT
    done
  done
done
unset TEA_B200_LIB
python - <<'PY'
import json
for l in open("gpurun_out/stat_minb.jsonl"):
    d = json.loads(l); r = d["roofline"]
    print(d["variant"], d["config"]["method"], d["config"]["mesh"], round(d["value"], 1), r["kernel_gbs"].get("stat"), d["clocks"]["sm_mhz"])
PY
