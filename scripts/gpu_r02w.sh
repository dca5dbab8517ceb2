for v in cur o1 o2 o3 o4 o5 cur o1; do
  printf "%s " $v; LNS_LIB=build/variants/liblns_$v.so timeout 300 python scripts/probe_batch.py C4:50:400 C4:49:400 C3:50:400 C2:148:2000 2>&1 | tail -4 | awk '{printf "%s %s  ", $1, $8}'; echo
  LNS_LIB=build/variants/liblns_$v.so timeout 300 python scripts/probe_single.py 2>&1 | tail -2 | tr '\n' ' '; echo
done
