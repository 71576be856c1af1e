# SpMV occupancy A/B (TEA_SPMV_MINB variants from tools/build_variants.py), interleaved (gpurun)
: > gpurun_out/spmv_minb.jsonl
for rep in 1 2; do
  for v in default spmv6 spmv8; do
    if [ $v = default ]; then unset TEA_B200_LIB; else export TEA_B200_LIB=build_variants/$v.so; fi
    for m in cg cppcg; do
      timeout 300 python bench.py --no-cpu --method $m --steps 3 | tail -1 | sed "s/^{/{\"variant\": \"$v\", /" >> gpurun_out/spmv_minb.jsonl
    done
  done
done
unset TEA_B200_LIB
