#!/bin/bash
# Bench lines for every method and the BASELINE configs (run under gpurun, 1 GPU).
# Usage: bash tools/bench_matrix.sh <out.jsonl>
OUT=${1:-gpurun_out/bench_matrix.jsonl}
: > $OUT
run() { timeout 600 python bench.py "$@" --no-cpu 2>/dev/null | tail -1 >> $OUT; }
run --method cppcg --n 4096 --steps 5 --warmup 3
run --method cppcg --n 4096 --steps 5 --warmup 3 --kform -1   # stored faces (A/B, §4.13)
run --method cg --n 4096 --steps 3 --warmup 3
run --method cg1 --n 4096 --steps 3 --warmup 3
run --method bjcg --n 4096 --steps 3 --warmup 3
run --method jacobi --n 4096 --steps 3 --warmup 3
run --method cheby --n 4096 --steps 3 --warmup 3
run --method cppcg --n 1024 --steps 10 --warmup 3
run --method cg --n 1024 --steps 10 --warmup 3
run --method cg --n 128 --steps 10 --warmup 3 --eps 1e-15
run --method cppcg --n 128 --steps 10 --warmup 3 --eps 1e-15
run --method cg --n 256 --nz 256 --steps 3 --warmup 3
run --method cppcg --n 4096 --steps 3 --warmup 3 --blocks 2x4 --halo-depth 2
run --method cppcg --n 4096 --steps 3 --warmup 3 --blocks 2x4 --halo-depth 10
run --method cppcg --n 4096 --steps 3 --warmup 3 --blocks 2x4 --halo-depth 11
run --method cppcg --n 4096 --steps 3 --warmup 3 --blocks 2x4 --halo-depth 11 --overlap 1
run --method cg --n 4096 --steps 3 --warmup 3 --blocks 2x4 --halo-depth 1
run --method cppcg --n 16384 --steps 1 --warmup 3 --max-iters 100000
run --method cppcg --n 16384 --steps 1 --warmup 3 --max-iters 100000 --blocks 2x4
run --method cppcg --n 256 --nz 256 --steps 3 --warmup 3
python - $OUT <<'PY'
import json, sys
for l in open(sys.argv[1]):
    try: d = json.loads(l)
    except Exception: continue
    r = d["roofline"]
    kf = '' if d['config'].get('kform', 'g').startswith('g') else ' [stored K]'
    print(f"{d['config']['workload'] + ' ' + d['config']['parallelism'] + kf:62s} {d['value']:9.1f} it/s  {d['time_to_solution_s']*1e3:9.2f} ms/step "
          f"its={d['iterations_per_step']:.0f} model={d['hbm_gbs_model']:.0f}GB/s dom={r['kernel']} "
          f"frac={r['frac']:.3f}")
PY
