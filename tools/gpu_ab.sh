#!/bin/bash
# Interleaved same-box A/B of library variants (gpurun): bench.py timed region with in-graph
# kernel timing. Usage: bash tools/gpu_ab.sh TAG "variant1 variant2 ..." "bench args" [reps]
# variant "default" = the in-tree library; others = build_variants/<name>.so
TAG=$1; VARS=$2; ARGS=$3; REPS=${4:-2}
OUT=gpurun_out/ab_$TAG.jsonl; : > $OUT
for rep in $(seq $REPS); do
  for v in $VARS; do
    if [ $v = default ]; then unset TEA_B200_LIB; else export TEA_B200_LIB=build_variants/$v.so; fi
    timeout 600 python bench.py --no-cpu --steps 10 --warmup 3 $ARGS | tail -1 | sed "s/^{/{\"variant\": \"$v\", /" >> $OUT
  done
done
unset TEA_B200_LIB
python - "$OUT" <<'PY'
import json, sys
for l in open(sys.argv[1]):
    try:
        d = json.loads(l)
    except Exception:
        print("bad line", l[:200]); continue
    r = d.get("roofline") or {}
    print(d["variant"], d["config"]["method"], d["config"]["mesh"], d["config"].get("parallelism"),
          round(d["value"], 1), "it/s", round(d["ms_per_step"], 2), "ms", r.get("kernel_avg_us"),
          "sm", d["clocks"]["sm_mhz"])
PY
