# ncu --set full of the two other views of k_search<3> on the round-2 kernel, summarised into
# gpurun_out/r02_ncu_k_search_{single,C5}.json (copy into profiles/): one C4 search of 1,000
# iterations on all SMs (the latency view) and the first C5 search launch (3 iterations).
SHA=$(python -c "from paper_conf_ipps_luongmt10_b200 import _build; print(_build.source_hash())")
cap() {  # name script skip units kernel-description
  timeout 900 ncu --set full --clock-control none --import-source on -k regex:k_search -s $3 -c 1 \
    -o gpurun_out/$1 -f python scripts/$2 > gpurun_out/$1.log 2>&1; echo ncu_$1=$?
  ncu -i gpurun_out/$1.ncu-rep --page raw --csv > gpurun_out/$1_raw.csv 2>/dev/null
  ncu -i gpurun_out/$1.ncu-rep --page source --csv --print-source sass > gpurun_out/$1_sass.csv 2>/dev/null
  python scripts/ncu_summary.py gpurun_out/$1_raw.csv gpurun_out/r02_ncu_k_search_$1.json --kernel "$5" \
    --capture "ncu --set full --clock-control none --import-source on -k regex:k_search -s $3 -c 1 python scripts/$2" \
    --source gpurun_out/$1_sass.csv --units $4 --source-sha "$SHA" > /dev/null; echo summary_$1=$?
  python scripts/sass_hot.py gpurun_out/$1_sass.csv $4 10 > gpurun_out/r02_k_search_$1_hot.txt 2>&1
  rm -f gpurun_out/$1_sass.csv gpurun_out/$1.ncu-rep
}
cap single profile_single.py 1 260130000 "k_search<3> one search: C4, 1,000 iterations on 148 CTAs (latency view)"
cap C5 profile_c5.py 0 535299072 "k_search<3> one search: C5 (1024 x 1024), 3 iterations on 148 CTAs"
