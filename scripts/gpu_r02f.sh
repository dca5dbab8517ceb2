# round-2 call F: slot-array exchange + pair-path trims vs HEAD; phase breakdown of the single search
timeout 1200 python -m pytest tests -m gpu -x -q > gpurun_out/pytest_gpu_f.log 2>&1; echo pytest=$?
tail -4 gpurun_out/pytest_gpu_f.log
for v in head cur; do
  lib=build/variants/liblns_$v.so; [ $v = cur ] && lib=paper_conf_ipps_luongmt10_b200/liblns.so
  echo "== $v"
  LNS_LIB=$lib timeout 300 python scripts/probe_batch.py C4:50:400 C4:50:400 C3:50:400 C2:148:2000 2>&1 | tail -4
  LNS_LIB=$lib timeout 300 python scripts/probe_single.py 2>&1 | tail -5
done
echo "== phases head"; LNS_PROF_LIB=build/variants/liblns_headprof.so timeout 300 python scripts/phases.py C4:148:1000 C3:148:1000 2>&1 | tail -20
echo "== phases cur"; timeout 300 python scripts/phases.py C4:148:1000 C3:148:1000 2>&1 | tail -20
