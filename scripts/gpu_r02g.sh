# round-2 call G: A/B head / head+2 planes / current (pair trims + 2 planes + plan step C split) / current 3 planes
timeout 1200 python -m pytest tests -m gpu -x -q > gpurun_out/pytest_gpu_g.log 2>&1; echo pytest=$?
tail -3 gpurun_out/pytest_gpu_g.log
for v in head head2p cur cur3 head; do
  lib=build/variants/liblns_$v.so; [ $v = cur ] && lib=paper_conf_ipps_luongmt10_b200/liblns.so
  echo "== $v"
  LNS_LIB=$lib timeout 300 python scripts/probe_batch.py C4:50:400 C4:50:400 C3:50:400 C2:148:2000 2>&1 | tail -4
  LNS_LIB=$lib timeout 300 python scripts/probe_single.py 2>&1 | tail -4
done
echo "== phases cur"; timeout 300 python scripts/phases.py C4:148:1000 C3:148:1000 2>&1 | tail -20
