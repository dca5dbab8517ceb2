# round-2 call D: GPU tests on the bitmap+ring tabu state; A/B of variants on the bench job
timeout 1500 python -m pytest tests -m gpu -x -q > gpurun_out/pytest_gpu_d.log 2>&1; echo pytest=$?
tail -15 gpurun_out/pytest_gpu_d.log
for v in base pf gen2; do
  echo "== $v"
  LNS_LIB=build/variants/liblns_$v.so timeout 300 python scripts/probe_batch.py C4:50:400 C4:50:400 C3:50:400 2>&1 | tail -3
done
echo "== base LNS_NO_BITS=1"
LNS_NO_BITS=1 LNS_LIB=build/variants/liblns_base.so timeout 300 python scripts/probe_batch.py C4:50:400 C4:50:400 2>&1 | tail -2
echo "== C5 single (bits) / (no bits)"
timeout 300 python scripts/probe_c5.py 2>&1 | tail -4
LNS_NO_BITS=1 timeout 300 python scripts/probe_c5.py 2>&1 | tail -4
