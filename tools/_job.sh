mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > /dev/null 2>&1
echo "== impl0"; TEA_TB_IMPL=0 timeout 300 python tools/tb_sweep.py --n 4096 --steps 5 --rows 0 2>&1 | tail -1
for v in regr regr3 regkx3 both both3; do
  echo "== $v"; TEA_TB_IMPL=2 TEA_B200_LIB=build_variants/$v.so timeout 300 python tools/tb_sweep.py --n 4096 --steps 5 --rows 0 2>&1 | tail -1
done
TEA_TB_IMPL=2 TEA_B200_LIB=build_variants/regkx3.so timeout 600 python -m pytest tests/test_gpu_parity.py -m gpu -x -q -k "fused" 2>&1 | tail -1
