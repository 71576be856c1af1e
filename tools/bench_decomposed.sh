OUT=gpurun_out/bench_new.jsonl; : > $OUT
run() { timeout 900 python bench.py "$@" --no-cpu 2>gpurun_out/bench_new_err.log | tail -1 >> $OUT; }
run --method cppcg --n 4096 --steps 3 --warmup 3 --blocks 2x4 --halo-depth 2
run --method cppcg --n 4096 --steps 3 --warmup 3 --blocks 2x4 --halo-depth 10
run --method cppcg --n 4096 --steps 3 --warmup 3 --blocks 2x4 --halo-depth 11
run --method cppcg --n 4096 --steps 3 --warmup 3 --blocks 2x4 --halo-depth 16
run --method cppcg --n 4096 --steps 3 --warmup 3 --blocks 1x2 --halo-depth 11
run --method cppcg --n 4096 --steps 3 --warmup 3 --blocks 2x2 --halo-depth 11
run --method cg --n 4096 --steps 3 --warmup 3 --blocks 2x4 --halo-depth 1
run --method cppcg --n 16384 --steps 1 --warmup 3 --blocks 2x4 --halo-depth 11
python - $OUT <<'PY'
import json, sys
for l in open(sys.argv[1]):
    try: d = json.loads(l)
    except Exception: continue
    r = d["roofline"]
    print(f"{d['config']['workload']:50s} {d['config']['parallelism']:45s} {d['value']:8.1f} it/s {d['time_to_solution_s']*1e3:9.1f} ms/step its={d['iterations_per_step']:.0f} dom={r['kernel']} frac={r['frac']:.3f} kms={r['kernel_ms']}")
PY
