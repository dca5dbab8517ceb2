# round-2 call J: next-row-word plane prefetch and record-loop unroll (A/B on the bench job)
for v in cur pp1 pp1u2 u2 cur; do
  echo "== $v"
  LNS_LIB=build/variants/liblns_$v.so timeout 300 python scripts/probe_batch.py C4:50:400 C4:50:400 C3:50:400 C2:148:2000 2>&1 | tail -4
  LNS_LIB=build/variants/liblns_$v.so timeout 300 python scripts/probe_single.py 2>&1 | tail -2
done
