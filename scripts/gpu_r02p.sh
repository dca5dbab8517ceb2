# round-2 call P: why is the batched instantiation slower? ncu of one bench step, cur vs split
for v in cur split; do
  LNS_LIB=build/variants/liblns_$v.so timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_search -s 1 -c 1 -o gpurun_out/bs_$v -f python scripts/profile_bench_step.py > gpurun_out/ncu_bs_$v.log 2>&1; echo ncu_$v=$?
  ncu -i gpurun_out/bs_$v.ncu-rep --page raw --csv > gpurun_out/bs_${v}_raw.csv 2>/dev/null
  ncu -i gpurun_out/bs_$v.ncu-rep --page source --csv --print-source sass > gpurun_out/bs_${v}_sass.csv 2>/dev/null
  python scripts/sass_hot.py gpurun_out/bs_${v}_sass.csv 5.2026e9 14 > gpurun_out/bs_${v}_hot.txt 2>&1
  rm -f gpurun_out/bs_${v}_sass.csv gpurun_out/bs_$v.ncu-rep
done
for v in split2; do
  echo "== $v"
  LNS_LIB=build/variants/liblns_$v.so timeout 300 python scripts/probe_batch.py C4:50:400 C4:50:400 C2:148:2000 2>&1 | tail -3
  LNS_LIB=build/variants/liblns_$v.so timeout 300 python scripts/probe_single.py 2>&1 | tail -4
done
