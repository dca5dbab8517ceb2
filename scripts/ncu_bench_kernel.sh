# one full ncu capture (source-level) of the bench kernel: k_search<3> on one bench step
timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_search -s 1 -c 1 -o gpurun_out/k_search_full -f python scripts/profile_bench_step.py > gpurun_out/ncu_full.log 2>&1; echo ncu=$?
ncu -i gpurun_out/k_search_full.ncu-rep --page raw --csv > gpurun_out/k_search_raw.csv 2>/dev/null
ncu -i gpurun_out/k_search_full.ncu-rep --page source --csv --print-source sass > gpurun_out/k_search_sass.csv 2>/dev/null
ls -la gpurun_out/k_search*
