# round-2 call I: GPU tests, bench-kernel capture of the current sources, the bench
timeout 1200 python -m pytest tests -m gpu -x -q > gpurun_out/pytest_gpu_i.log 2>&1; echo pytest=$?
tail -3 gpurun_out/pytest_gpu_i.log
bash scripts/capture_bench_kernel.sh
timeout 600 python bench.py > gpurun_out/bench_i.log 2>&1; echo bench=$?
tail -c 1200 gpurun_out/bench_i.log
head -c 700 gpurun_out/bench_i.log
