# round-2 call L: flip-set keys (no unranking after the exchange) + records overlapped with the row placement
timeout 1200 python -m pytest tests -m gpu -x -q > gpurun_out/pytest_gpu_l.log 2>&1; echo pytest=$?
tail -3 gpurun_out/pytest_gpu_l.log
for v in cur2 cur; do
  lib=build/variants/liblns_$v.so; [ $v = cur2 ] && lib=paper_conf_ipps_luongmt10_b200/liblns.so
  echo "== $v"
  LNS_LIB=$lib timeout 300 python scripts/probe_batch.py C4:50:400 C4:50:400 C3:50:400 C2:148:2000 2>&1 | tail -4
  LNS_LIB=$lib timeout 300 python scripts/probe_single.py 2>&1 | tail -4
done
echo "== phases"; timeout 300 python scripts/phases.py C4:148:1000 2>&1 | tail -13
