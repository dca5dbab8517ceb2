# round-2 call X: GPU tests, capture, bench on the split kernel (batched / single-search instantiations)
timeout 1200 python -m pytest tests -m gpu -x -q > gpurun_out/pytest_gpu_x.log 2>&1; echo pytest=$?
tail -3 gpurun_out/pytest_gpu_x.log
bash scripts/capture_bench_kernel.sh
timeout 600 python bench.py > gpurun_out/bench_x.log 2>&1; echo bench=$?
grep '^{' gpurun_out/bench_x.log | head -c 600
echo "== phases"; timeout 300 python scripts/phases.py C4:148:1000 2>&1 | tail -11
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/launches_bench_x.csv python bench.py --steps 2 --warmup 3 --no-cpu-baseline > gpurun_out/bench_under_ncu_x.log 2>&1; echo ncu_launches=$?
