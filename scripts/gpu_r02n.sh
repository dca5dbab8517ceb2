# round-2 call N: bisect the batched regression (hw = HEAD + window constants in warp 1; noenc = current without flip-set keys)
for v in cur hw noenc cur2; do
  echo "== $v"
  LNS_LIB=build/variants/liblns_$v.so timeout 300 python scripts/probe_batch.py C4:50:400 C4:50:400 2>&1 | tail -2
  LNS_LIB=build/variants/liblns_$v.so timeout 300 python scripts/probe_single.py 2>&1 | tail -2
done
timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_search -s 1 -c 1 -o gpurun_out/k_single_full -f python scripts/profile_single.py > gpurun_out/ncu_single.log 2>&1; echo ncu=$?
ncu -i gpurun_out/k_single_full.ncu-rep --page source --csv --print-source sass > gpurun_out/k_single_sass.csv 2>/dev/null
python scripts/sass_hot.py gpurun_out/k_single_sass.csv 0 40 > gpurun_out/k_single_hot.txt 2>&1
rm -f gpurun_out/k_single_sass.csv gpurun_out/k_single_full.ncu-rep
