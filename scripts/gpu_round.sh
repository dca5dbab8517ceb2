# one gpurun call: GPU parity tests, the bench, and (NCU=1) one full ncu capture of the bench kernel
timeout 900 python -m pytest tests -m gpu -x -q > gpurun_out/pytest_gpu.log 2>&1; echo pytest=$?
tail -15 gpurun_out/pytest_gpu.log
timeout 400 python bench.py ${BENCH_ARGS:-} > gpurun_out/bench.log 2>&1; echo bench=$?
tail -c 1500 gpurun_out/bench.log
if [ "${NCU:-0}" = 1 ]; then
  timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_search -s 1 -c 1 -o gpurun_out/k_search_full -f python scripts/profile_bench_step.py > gpurun_out/ncu_full.log 2>&1; echo ncu=$?
  ncu -i gpurun_out/k_search_full.ncu-rep --page raw --csv > gpurun_out/k_search_raw.csv 2>/dev/null
  ncu -i gpurun_out/k_search_full.ncu-rep --page source --csv --print-source sass > gpurun_out/k_search_sass.csv 2>/dev/null
fi
