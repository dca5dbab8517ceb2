# ncu --set full of the bench kernel for each build given as NAME=LIBPATH (A/B of kernel variants)
for spec in "$@"; do
  name=${spec%%=*}; lib=${spec#*=}
  LNS_LIB=$lib timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_search -s 1 -c 1 \
    -o gpurun_out/ab_$name -f python scripts/profile_bench_step.py > gpurun_out/ab_$name.log 2>&1; echo ncu_$name=$?
  ncu -i gpurun_out/ab_$name.ncu-rep --page raw --csv > gpurun_out/ab_${name}_raw.csv 2>/dev/null
  ncu -i gpurun_out/ab_$name.ncu-rep --page source --csv --print-source sass > gpurun_out/ab_${name}_sass.csv 2>/dev/null
  python scripts/sass_hot.py gpurun_out/ab_${name}_sass.csv 5.2026e9 14 > gpurun_out/ab_${name}_hot.txt 2>&1
  rm -f gpurun_out/ab_${name}_sass.csv gpurun_out/ab_$name.ncu-rep
done
