# A/B of experimental builds (build/variants/liblns_<name>.so) on the bench job, C3 batches, C5 and the single searches
for v in "$@"; do
  echo "== $v"
  LNS_LIB=build/variants/liblns_$v.so timeout 300 python scripts/probe_batch.py C4:50:400 C4:50:400 C3:50:400 2>&1 | tail -3
  LNS_LIB=build/variants/liblns_$v.so timeout 300 python scripts/probe_c5.py 2>&1 | tail -2
  LNS_LIB=build/variants/liblns_$v.so timeout 300 python scripts/probe_single.py 2>&1 | tail -4
done
