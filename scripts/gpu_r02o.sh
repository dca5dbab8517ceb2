# round-2 call O: k_search split into batched / single-search instantiations
for v in cur split cur split; do
  echo "== $v"
  LNS_LIB=build/variants/liblns_$v.so timeout 300 python scripts/probe_batch.py C4:50:400 C4:50:400 C3:50:400 C2:148:2000 2>&1 | tail -4
  LNS_LIB=build/variants/liblns_$v.so timeout 300 python scripts/probe_single.py 2>&1 | tail -4
done
LNS_LIB=build/variants/liblns_split.so timeout 300 python scripts/probe_c5.py 2>&1 | tail -2
