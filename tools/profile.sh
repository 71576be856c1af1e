#!/bin/bash
# Run on the GPU box (gpurun): launch list + ncu --set full captures of the hot kernels.
# Usage: bash tools/profile.sh <tag> [n]
set -x
TAG=${1:-r01}; N=${2:-4096}
OUT=gpurun_out/prof_$TAG; mkdir -p $OUT
python -c "import __graft_entry__ as g; g.build()" > $OUT/build.log 2>&1
# 1) launch list of the bench command (cold-cache, serialised: compare shares). Loop mode 2
#    (eager launches): ncu does not profile kernels of graphs with WHILE nodes, and the
#    chunked graphs of mode 1 listed only the first fused pass (r01h, r01j).
timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none -c 3000 --csv \
   --log-file $OUT/launches.csv python bench.py --n $N --steps 1 --warmup 3 --no-cpu \
   --loop-mode 2 > $OUT/bench_under_ncu.log 2>&1
# 1b) the same list with the L2 left as the previous kernel left it (--cache-control none):
#    what the bench's in-graph timing sees (write-back of the predecessor's dirty lines)
timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none --cache-control none \
   -c 3000 --csv --log-file $OUT/launches_warm.csv python bench.py --n $N --steps 1 --warmup 3 \
   --no-cpu --loop-mode 2 > $OUT/bench_under_ncu_warm.log 2>&1
# 2) full sets: the fused Chebyshev passes of the first outer iterations (skip the two
#    restart passes) and two SpMVs of the PCG phase
timeout 900 ncu --set full --clock-control none --import-source on \
   -k regex:"k_cheb_tb" -s 2 -c 4 -o $OUT/full_tb \
   python tools/kernel_sweep.py --n $N --once --iters 40 > $OUT/full_tb.log 2>&1
timeout 900 ncu --set full --clock-control none --import-source on \
   -k regex:"k_spmv" -s 40 -c 2 -o $OUT/full_spmv \
   python tools/kernel_sweep.py --n $N --once --iters 40 > $OUT/full_spmv.log 2>&1
ls -la $OUT
