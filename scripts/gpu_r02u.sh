for v in cur split3; do
  LNS_LIB=build/variants/liblns_$v.so timeout 900 ncu --cache-control none --clock-control none -k regex:k_search -s 1 -c 1 --section WarpStateStats --section SchedulerStats --section ComputeWorkloadAnalysis --section InstructionStats --metrics gpu__time_duration.sum,smsp__average_warps_issue_stalled_no_instruction_per_issue_active.ratio,sm__inst_executed_pipe_xu.avg.pct_of_peak_sustained_active --csv --page raw python scripts/profile_bench_step.py > gpurun_out/u_$v.csv 2>&1; echo $v=$?
done
