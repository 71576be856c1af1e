mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build(); g.smoke()" > gpurun_out/smoke2.log 2>&1
timeout 600 python -m pytest tests/test_gpu_parity.py -m gpu -x -q -k kform > gpurun_out/kform_tests.log 2>&1
for kf in 1 -1 1 -1; do timeout 300 python bench.py --no-cpu --kform $kf | tail -1 >> gpurun_out/kform_ab.jsonl; done
for kf in 1 -1; do timeout 300 python bench.py --no-cpu --method cg --steps 3 --kform $kf | tail -1 >> gpurun_out/kform_ab.jsonl; done
timeout 900 python -m pytest tests -m gpu -x -q > gpurun_out/gpu_tests2.log 2>&1
