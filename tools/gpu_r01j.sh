# round-1j GPU pass (run under gpurun): smoke, kform bitwise tests, the full GPU suite, the
# default bench line, then the launch list + ncu full sets of the hot kernels (tools/profile.sh)
mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build(); g.smoke()" > gpurun_out/smoke4.log 2>&1
timeout 900 python -m pytest tests/test_gpu_parity.py -m gpu -q -k kform > gpurun_out/kform_tests.log 2>&1
timeout 900 python -m pytest tests -m gpu -q > gpurun_out/gpu_tests4.log 2>&1
timeout 600 python bench.py > gpurun_out/bench_r01j.log 2>&1
bash tools/profile.sh r01j > gpurun_out/profile_r01j.log 2>&1
