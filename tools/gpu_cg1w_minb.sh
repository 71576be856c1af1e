#!/bin/bash
# k_cg1_w occupancy A/B (TEA_CG1W_MINB), single-reduction CPPCG 4096^2 and 256^3, interleaved x2 (gpurun)
OUT=gpurun_out/cg1w_minb.jsonl; : > $OUT
for rep in 1 2; do
  for v in default w7 w8; do
    if [ $v = default ]; then unset TEA_B200_LIB; else export TEA_B200_LIB=build_variants/$v.so; fi
    for args in "--method cppcg1" "--n 256 --nz 256 --method cppcg1"; do
      timeout 300 python bench.py --no-cpu --steps 3 $args | tail -1 | sed "s/^{/{\"variant\": \"$v\", /" >> $OUT
    done
  done
done
unset TEA_B200_LIB
python - <<'PY'
import json
for l in open("gpurun_out/cg1w_minb.jsonl"):
    d = json.loads(l); r = d["roofline"]
    print(d["variant"], d["config"]["mesh"], round(d["value"], 1), r["kernel_gbs"], d["clocks"]["sm_mhz"])
PY
