# round-2 call R: batched instantiation without the placement overlap (split3)
for rep in 1 2; do
  for v in cur split2 split3; do
    printf "%s %s " $rep $v
    LNS_LIB=build/variants/liblns_$v.so timeout 300 python scripts/probe_batch.py C4:50:400 2>&1 | tail -1 | awk '{print $5, $8}'
  done
done
LNS_LIB=build/variants/liblns_split3.so timeout 300 python scripts/probe_batch.py C3:50:400 C2:148:2000 2>&1 | tail -2
LNS_LIB=build/variants/liblns_split3.so timeout 300 python scripts/probe_single.py 2>&1 | tail -4
