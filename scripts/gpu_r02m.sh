# round-2 call M: which single-search change costs the batched job: placement overlap (po0 = off), spin back-off
for v in cur cur2 po0 sl50 sl200 cur2; do
  echo "== $v"
  LNS_LIB=build/variants/liblns_$v.so timeout 300 python scripts/probe_batch.py C4:50:400 C4:50:400 C3:50:400 2>&1 | tail -3
  LNS_LIB=build/variants/liblns_$v.so timeout 300 python scripts/probe_single.py 2>&1 | tail -3
done
