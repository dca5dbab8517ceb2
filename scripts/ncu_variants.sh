export PYTHONPATH=$PWD
timeout 300 ncu --set full --clock-control none --import-source on -k regex:k_bqp_eval -s 1 -c 1 -o gpurun_out/bqp_full -f python scripts/profile_bqp.py > gpurun_out/ncu_bqp.log 2>&1; echo ncu_bqp=$?
ncu -i gpurun_out/bqp_full.ncu-rep --page raw --csv > gpurun_out/bqp_raw.csv 2>/dev/null
timeout 300 ncu --set full --clock-control none --import-source on -k regex:k_gen -s 1 -c 1 -o gpurun_out/kgen_full -f python scripts/profile_kgen.py > gpurun_out/ncu_kgen.log 2>&1; echo ncu_kgen=$?
ncu -i gpurun_out/kgen_full.ncu-rep --page raw --csv > gpurun_out/kgen_raw.csv 2>/dev/null
ncu -i gpurun_out/kgen_full.ncu-rep --page source --csv --print-source sass > gpurun_out/kgen_sass.csv 2>/dev/null
rm -f gpurun_out/*.ncu-rep
ls -la gpurun_out/
