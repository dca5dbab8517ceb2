# round-2 call E: pair-path overhead trims (strict per-half compare, cached tabu words), 2 vs 3 planes
timeout 900 python -m pytest tests -m gpu -x -q -k "batch or restarts or trajectory or pool or bench or eval_all" > gpurun_out/pytest_gpu_e.log 2>&1; echo pytest=$?
tail -4 gpurun_out/pytest_gpu_e.log
for v in base threeplanes; do
  echo "== $v"
  LNS_LIB=build/variants/liblns_$v.so timeout 300 python scripts/probe_batch.py C4:50:400 C4:50:400 C3:50:400 C2:148:2000 2>&1 | tail -4
done
