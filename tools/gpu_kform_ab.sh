# kform A/B on one GPU (run under gpurun): kform tests, then 4096^2 CPPCG / CG / CG1 / CPPCG1 /
# Jacobi bench lines with the faces on the fly (1) and stored (-1), interleaved
mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build(); g.smoke()" > gpurun_out/smoke3.log 2>&1
timeout 900 python -m pytest tests/test_gpu_parity.py -m gpu -x -q -k kform > gpurun_out/kform_tests.log 2>&1
: > gpurun_out/kform_ab.jsonl
for m in cppcg cg cg1 cppcg1 jacobi bjcg; do
  for kf in 1 -1; do timeout 300 python bench.py --no-cpu --method $m --steps 3 --kform $kf | tail -1 >> gpurun_out/kform_ab.jsonl; done
done
timeout 900 python -m pytest tests -m gpu -x -q > gpurun_out/gpu_tests3.log 2>&1
