# round-2 call A: integer-pipe peaks (microbenchmark + ncu pipe metrics) and the GPU tests
mkdir -p gpurun_out build
nvcc -gencode arch=compute_100a,code=sm_100a -O3 -lineinfo -o build/int_peaks scripts/int_peaks.cu && \
  timeout 120 build/int_peaks > gpurun_out/int_peaks.json 2> gpurun_out/int_peaks.err; echo int_peaks=$?
cat gpurun_out/int_peaks.json
timeout 300 ncu --clock-control none --metrics sm__inst_executed_pipe_alu.avg.peak_sustained,sm__inst_executed_pipe_fma.avg.peak_sustained,sm__inst_executed_pipe_fmaheavy.avg.peak_sustained,sm__inst_executed_pipe_xu.avg.peak_sustained,sm__inst_executed_pipe_lsu.avg.peak_sustained,smsp__issue_active.avg.peak_sustained,sm__inst_executed_pipe_alu.avg.pct_of_peak_sustained_active,sm__inst_executed_pipe_fma.avg.pct_of_peak_sustained_active,sm__inst_executed_pipe_xu.avg.pct_of_peak_sustained_active,smsp__issue_active.avg.pct_of_peak_sustained_active,sm__cycles_elapsed.avg.per_second --csv build/int_peaks > gpurun_out/int_peaks_ncu.csv 2>&1; echo ncu=$?
timeout 1500 python -m pytest tests -m gpu -x -q -k "not golden" > gpurun_out/pytest_gpu.log 2>&1; echo pytest=$?
tail -25 gpurun_out/pytest_gpu.log
