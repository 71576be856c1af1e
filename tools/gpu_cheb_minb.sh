#!/bin/bash
# per-step Chebyshev kernels (k_cheb) occupancy A/B: TEA_CHEB_MINB variants, interleaved x2 (gpurun)
OUT=gpurun_out/cheb_minb.jsonl; : > $OUT
for rep in 1 2; do
  for v in default ch6 ch7; do
    if [ $v = default ]; then unset TEA_B200_LIB; else export TEA_B200_LIB=build_variants/$v.so; fi
    for args in "--n 256 --nz 256 --method cppcg" "--method cppcg --tb-steps 1"; do
      timeout 300 python bench.py --no-cpu --steps 3 $args | tail -1 | sed "s/^{/{\"variant\": \"$v\", /" >> $OUT
    done
  done
done
unset TEA_B200_LIB
python - <<'PY'
import json
for l in open("gpurun_out/cheb_minb.jsonl"):
    d = json.loads(l); r = d["roofline"]
    print(d["variant"], d["config"]["mesh"], round(d["value"], 1), {k: v for k, v in r["kernel_gbs"].items() if "cheb" in k}, d["clocks"]["sm_mhz"])
PY
