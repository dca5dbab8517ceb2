# A/B of variant builds on the bench job (C4 batched) and C3 batched: gpu_ab.sh NAME...
for v in "$@"; do
  echo "== $v"; LNS_LIB=build/variants/liblns_$v.so timeout 300 python scripts/probe_batch.py C4:50:400 C4:50:400 C3:50:400 2>&1 | tail -3
done
