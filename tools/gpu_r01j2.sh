# launch list in eager mode (all kernels visible to ncu), bench matrix, sanitizers (gpurun)
mkdir -p gpurun_out/prof_r01j2
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/prof_r01j2/build.log 2>&1
timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none -c 3000 --csv \
   --log-file gpurun_out/prof_r01j2/launches.csv python bench.py --n 4096 --steps 1 --warmup 3 --no-cpu \
   --loop-mode 2 > gpurun_out/prof_r01j2/bench_under_ncu.log 2>&1
bash tools/bench_matrix.sh gpurun_out/bench_matrix_r01j.jsonl > gpurun_out/bench_matrix_r01j.txt 2>&1
mkdir -p gpurun_out/san
for tool in memcheck initcheck racecheck; do
  timeout 900 compute-sanitizer --tool $tool --error-exitcode 9 python tools/sanitize.py > gpurun_out/san/$tool.log 2>&1; echo "$tool rc=$?" >> gpurun_out/san/summary.txt
done
