#!/bin/bash
# r01k: 3D SpMV evidence -- bench lines for 256^3 CG/CPPCG and one ncu --set full capture
# of the 3D SpMV (loop mode 2 so ncu sees the launches).
OUT=gpurun_out/r01k3d; mkdir -p $OUT
for m in cg cppcg; do
  timeout 300 python bench.py --n 256 --nz 256 --method $m --no-cpu > $OUT/bench_$m.json 2> $OUT/bench_$m.err
done
timeout 600 ncu --set full --clock-control none --import-source on -k regex:"k_spmv" -s 30 -c 1 \
   -o $OUT/full_spmv3d python bench.py --n 256 --nz 256 --method cg --steps 1 --warmup 3 \
   --no-cpu --loop-mode 2 > $OUT/ncu.log 2>&1
ncu -i $OUT/full_spmv3d.ncu-rep --page raw --csv > $OUT/full_spmv3d_raw.csv 2>/dev/null
ncu -i $OUT/full_spmv3d.ncu-rep --page details --csv > $OUT/full_spmv3d_details.csv 2>/dev/null
ls -la $OUT; cat $OUT/bench_*.json
