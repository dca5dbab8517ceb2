# round artifacts in one gpurun call: GPU tests, smoke, bench (N=1), the reference arm, an ncu
# launch list of the bench command and one full ncu capture of the bench kernel
timeout 900 python -m pytest tests -m gpu -x -q > gpurun_out/pytest_gpu.log 2>&1; echo pytest=$?
tail -3 gpurun_out/pytest_gpu.log
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/smoke.log 2>&1; echo smoke=$?
timeout 400 python bench.py > gpurun_out/bench.log 2>&1; echo bench=$?
timeout 400 python bench.py --impl reference > gpurun_out/bench_reference.log 2>&1; echo ref=$?
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none -c 400 --csv --log-file gpurun_out/launches_bench.csv python bench.py --steps 2 --warmup 3 --no-cpu-baseline --no-single --no-c5 --no-ubqp > gpurun_out/bench_under_ncu.log 2>&1; echo launches=$?
bash scripts/ncu_bench_kernel.sh
rm -f gpurun_out/*.ncu-rep  # the CSV exports above are what comes back (gpurun_out is capped at 64 MiB)
