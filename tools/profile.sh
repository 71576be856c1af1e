#!/bin/bash
# Run on the GPU box (gpurun): launch list + ncu --set full captures of the hot kernels.
# Usage: bash tools/profile.sh <tag> [n]
set -x
TAG=${1:-r01}; N=${2:-4096}
OUT=gpurun_out/prof_$TAG; mkdir -p $OUT
python -c "import __graft_entry__ as g; g.build()" > $OUT/build.log 2>&1
# 1) launch list of the bench command (cold-cache, serialised: compare shares)
timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none -c 3000 --csv \
   --log-file $OUT/launches.csv python bench.py --n $N --steps 1 --warmup 3 --no-cpu --loop-mode 1 > $OUT/bench_under_ncu.log 2>   --log-file $OUT/launches.csv python bench.py --n $N --steps 1 --warmup 3 --no-cpu > $OUT/bench_under_ncu.log 2>&11
# 2) full sets of the hot kernels (eager solve: 30 presteps + ~10 outer)
timeout 900 ncu --set full --clock-control none --import-source on \
   -k regex:"k_cheb|k_spmv|k_update|k_residual" -s 60 -c 10 -o $OUT/full \
   python tools/kernel_sweep.py --n $N --once --iters 45 > $OUT/full.log 2>&1
ls -la $OUT
