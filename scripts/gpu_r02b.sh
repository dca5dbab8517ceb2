# round-2 call B: integer peaks (per-SM clock), C5 golden test, the bench-kernel capture, the bench
mkdir -p gpurun_out build
nvcc -gencode arch=compute_100a,code=sm_100a -O3 -lineinfo -o build/int_peaks scripts/int_peaks.cu && \
  timeout 120 build/int_peaks > gpurun_out/int_peaks.json 2> gpurun_out/int_peaks.err; echo int_peaks=$?
cat gpurun_out/int_peaks.json; cp gpurun_out/int_peaks.json profiles/int_peaks.json
timeout 900 python -m pytest tests -m gpu -x -q -k "golden" > gpurun_out/pytest_golden.log 2>&1; echo pytest=$?
tail -3 gpurun_out/pytest_golden.log
bash scripts/capture_bench_kernel.sh
timeout 600 python bench.py > gpurun_out/bench.log 2>&1; echo bench=$?
tail -c 3000 gpurun_out/bench.log
timeout 120 python bench.py --gpus 2 > gpurun_out/bench_gpus2.log 2>&1; echo bench_gpus2=$?
cat gpurun_out/bench_gpus2.log | tail -2
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/launches_bench.csv python bench.py --steps 2 --warmup 3 --no-cpu-baseline > gpurun_out/bench_under_ncu.log 2>&1; echo ncu_launches=$?
