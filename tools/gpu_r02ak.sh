#!/bin/bash
# programmatic dependent launch of the SpMV and the fused passes (TEA_PDL=1): bitwise check,
# parity subset, interleaved A/B on the headline and 1024^2
mkdir -p gpurun_out
TEA_PDL=1 python tools/dump_u.py /tmp/u_pdl.npz > gpurun_out/dump_ak.log 2>&1; echo "dump pdl rc=$?"
python tools/dump_u.py /tmp/u_nopdl.npz >> gpurun_out/dump_ak.log 2>&1
python - <<'PY'
import numpy as np
a = np.load("/tmp/u_pdl.npz"); b = np.load("/tmp/u_nopdl.npz")
print({k: ("bitwise" if np.array_equal(a[k], b[k]) else "DIFF") for k in a.files})
PY
tail -3 gpurun_out/dump_ak.log | cut -c1-300
TEA_PDL=1 timeout 1200 python -m pytest tests/test_gpu_parity.py tests/test_gpu_fullsize.py -m gpu -q -x -k "fused or converged or cppcg1f or multiblock or 1024 or loop_modes" > gpurun_out/pytest_pdl.log 2>&1; echo "pytest pdl rc=$?"; tail -2 gpurun_out/pytest_pdl.log
OUT=gpurun_out/ab_pdl.jsonl; : > $OUT
for rep in 1 2 3; do
  for v in off on; do
    if [ $v = on ]; then export TEA_PDL=1; else unset TEA_PDL; fi
    timeout 600 python bench.py --no-cpu --steps 10 --warmup 3 | tail -1 | sed "s/^{/{\"variant\": \"pdl_$v\", /" >> $OUT
    timeout 600 python bench.py --no-cpu --no-variants --n 1024 --steps 10 --warmup 3 | tail -1 | sed "s/^{/{\"variant\": \"pdl_$v\", /" >> $OUT
  done
done
unset TEA_PDL
python - <<'PY'
import json
for l in open("gpurun_out/ab_pdl.jsonl"):
    d = json.loads(l); r = d.get("roofline") or {}; v = d.get("variants", {}).get("cppcg1f", {})
    print(d["variant"], d["config"]["mesh"][0], round(d["value"], 1), round(r.get("kernel_time_of_step", 0), 4), r.get("kernel_avg_us"), d["clocks"]["sm_mhz"], "| 1f", round(v.get("value", 0), 1))
PY
