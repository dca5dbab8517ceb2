# ncu --set full of the bench kernel (k_search<3>, one bench step = 50 C4 searches x 400 iterations),
# summarised with the source hash of the build: gpurun_out/ncu_k_search_bench.json, also copied to
# profiles/ on the box so that a bench.py run in the same call accepts it (bench.py refuses a
# capture of other sources). Copy gpurun_out/ncu_k_search_bench.json into profiles/ afterwards.
SHA=$(python -c "from paper_conf_ipps_luongmt10_b200 import _build; print(_build.source_hash())")
timeout 900 ncu --set full --clock-control none --import-source on -k regex:k_search -s 1 -c 1 \
  -o gpurun_out/k_search_full -f python scripts/profile_bench_step.py > gpurun_out/ncu_full.log 2>&1; echo ncu=$?
ncu -i gpurun_out/k_search_full.ncu-rep --page raw --csv > gpurun_out/k_search_raw.csv 2>/dev/null
ncu -i gpurun_out/k_search_full.ncu-rep --page source --csv --print-source sass > gpurun_out/k_search_sass.csv 2>/dev/null
python scripts/ncu_summary.py gpurun_out/k_search_raw.csv gpurun_out/ncu_k_search_bench.json \
  --kernel "k_search<3> batched: one bench step = 50 C4 searches x 400 iterations" \
  --capture "ncu --set full --clock-control none --import-source on -k regex:k_search -s 1 -c 1 python scripts/profile_bench_step.py" \
  --source gpurun_out/k_search_sass.csv --units 5202600000 --source-sha "$SHA" > /dev/null && \
  cp gpurun_out/ncu_k_search_bench.json profiles/ncu_k_search_bench.json; echo summary=$?
python scripts/sass_hot.py gpurun_out/k_search_sass.csv 5.2026e9 12 > gpurun_out/k_search_hot.txt 2>&1
rm -f gpurun_out/k_search_sass.csv
