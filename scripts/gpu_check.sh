# GPU tests, smoke, bench and the reference arm on the current build (logs in gpurun_out/)
timeout 1500 python -m pytest tests -m gpu -x -q > gpurun_out/pytest_gpu.log 2>&1; echo pytest=$?
tail -2 gpurun_out/pytest_gpu.log
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/smoke.log 2>&1; echo smoke=$?
timeout 600 python bench.py > gpurun_out/bench.log 2>&1; echo bench=$?
grep '^{' gpurun_out/bench.log | head -c 400; echo
timeout 600 python bench.py --impl reference > gpurun_out/bench_ref.log 2>&1; echo ref=$?
grep '^{' gpurun_out/bench_ref.log | head -c 300
