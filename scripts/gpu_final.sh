# end-of-round artifacts on the current build: re-capture of the bench kernel (ncu --set full, hash
# of these sources), GPU tests, smoke, bench, reference arm, and the ncu launch list of the bench
bash scripts/capture_bench_kernel.sh
bash scripts/gpu_check.sh
timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none -c 400 --csv --log-file gpurun_out/launches_bench.csv \
  python bench.py --steps 2 --warmup 3 --no-cpu-baseline > gpurun_out/bench_under_ncu.log 2>&1; echo launches=$?
python scripts/launch_summary.py gpurun_out/launches_bench.csv "ncu --metrics gpu__time_duration.sum --clock-control none -c 400 python bench.py --steps 2 --warmup 3 --no-cpu-baseline (round 2, final kernel)" > gpurun_out/launches_summary.txt 2>&1; echo summary=$?
rm -f gpurun_out/*.ncu-rep
