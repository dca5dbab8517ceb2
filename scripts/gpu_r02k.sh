# round-2 call K: finer single-search phases; C5 DRAM traffic per launch with the bitmap tabu state
echo "== phases"; timeout 300 python scripts/phases.py C4:148:1000 C3:148:1000 2>&1 | tail -26
timeout 600 ncu --clock-control none -k regex:k_search --metrics dram__bytes_read.sum,dram__bytes_write.sum,gpu__time_duration.sum --csv python scripts/profile_c5.py > gpurun_out/ncu_c5_dram.csv 2>&1; echo ncu=$?
grep -v "^==PROF" gpurun_out/ncu_c5_dram.csv | tail -8
