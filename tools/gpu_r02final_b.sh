#!/bin/bash
# round 2 final pass B: the driver's bench commands (reference arm first, then ours), clocks
mkdir -p gpurun_out
timeout 1200 python bench.py --impl reference --steps 20 --warmup 5 > gpurun_out/ref_final.log 2>&1; echo "ref rc=$?"; tail -1 gpurun_out/ref_final.log
timeout 1200 python bench.py --steps 20 --warmup 5 > gpurun_out/bench_final.log 2>&1; echo "bench rc=$?"; tail -1 gpurun_out/bench_final.log
timeout 600 python bench.py > gpurun_out/bench_default.log 2>&1; echo "bench default rc=$?"; tail -1 gpurun_out/bench_default.log | cut -c1-300
