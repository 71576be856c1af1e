#!/bin/bash
# single-reduction CG occupancy A/B (TEA_CG1_MINB variants), 4096^2 and 256^3, interleaved x2 (gpurun)
OUT=gpurun_out/cg1_minb.jsonl; : > $OUT
for rep in 1 2; do
  for v in default cg1m4 cg1m5; do
    if [ $v = default ]; then unset TEA_B200_LIB; else export TEA_B200_LIB=build_variants/$v.so; fi
    timeout 300 python bench.py --no-cpu --method cg1 --steps 3 | tail -1 | sed "s/^{/{\"variant\": \"$v\", /" >> $OUT
    timeout 300 python bench.py --no-cpu --n 256 --nz 256 --method cg1 --steps 5 | tail -1 | sed "s/^{/{\"variant\": \"$v\", /" >> $OUT
  done
done
unset TEA_B200_LIB
python - <<'PY'
import json
for l in open("gpurun_out/cg1_minb.jsonl"):
    d = json.loads(l); r = d["roofline"]
    print(d["variant"], d["config"]["mesh"], round(d["value"], 1), r["kernel_gbs"], d["clocks"]["sm_mhz"])
PY
