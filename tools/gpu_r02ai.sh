#!/bin/bash
# first-pass staging depth 6 vs 5 (later passes 5), same box, 3 interleaved reps + ncu launch times
mkdir -p gpurun_out
bash tools/gpu_ab.sh cpa6 "default cpa6" "--no-variants" 3
for v in default cpa6; do
  if [ $v = default ]; then unset TEA_B200_LIB; else export TEA_B200_LIB=build_variants/$v.so; fi
  timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none -k regex:k_cheb_tb -c 40 --csv \
    python tools/kernel_sweep.py --n 4096 --once --iters 40 > gpurun_out/ncu_cpa_$v.csv 2>/dev/null
  python - "$v" <<'PY'
import csv, io, sys, collections
txt = open(f"gpurun_out/ncu_cpa_{sys.argv[1]}.csv").read(); i = txt.find('"ID"')
rows = list(csv.reader(io.StringIO(txt[i:]))); h = rows[0]
ki, vi = h.index("Kernel Name"), h.index("Metric Value")
agg = collections.defaultdict(list)
for r in rows[1:]:
    if len(r) > vi: agg[r[ki].split("(")[0]].append(float(r[vi].replace(",", "")))
for k, v in agg.items(): print(sys.argv[1], k, len(v), round(sum(v) / len(v) / 1e3, 1), "us")
PY
done
unset TEA_B200_LIB
