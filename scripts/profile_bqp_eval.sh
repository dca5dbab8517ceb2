# ncu --set full of one UBQP eval launch (k = 3, n = 500) inside the search loop, summarised
timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_bqp_eval -s 1 -c 1 \
  -o gpurun_out/bqp_eval -f python scripts/profile_bqp.py > gpurun_out/ncu_bqp.log 2>&1; echo ncu=$?
ncu -i gpurun_out/bqp_eval.ncu-rep --page raw --csv > gpurun_out/bqp_eval_raw.csv 2>/dev/null
ncu -i gpurun_out/bqp_eval.ncu-rep --page source --csv --print-source sass > gpurun_out/bqp_eval_sass.csv 2>/dev/null
python scripts/ncu_summary.py gpurun_out/bqp_eval_raw.csv gpurun_out/r02_ncu_k_bqp_eval_k3.json \
  --kernel "k_bqp_eval<3>: UBQP n = 500, one eval launch of the search loop (2.07e7 neighbours)" \
  --capture "ncu --set full --clock-control none --import-source on -k regex:k_bqp_eval -s 1 -c 1 python scripts/profile_bqp.py" \
  --source gpurun_out/bqp_eval_sass.csv --units 20708500 > /dev/null; echo summary=$?
rm -f gpurun_out/bqp_eval.ncu-rep gpurun_out/bqp_eval_sass.csv
