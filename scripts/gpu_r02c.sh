# round-2 call C: A/B of neighbours-per-thread (PK_NB) x threads-per-CTA (LNS_NT) variants on the bench job
for v in nb2 nb4 nt512nb2 nt512nb4 nt512nb6 nt512nb8 nt768nb4; do
  echo "== $v"
  LNS_LIB=build/variants/liblns_$v.so timeout 300 python scripts/probe_batch.py C4:50:400 C4:50:400 C3:50:400 2>&1 | tail -3
done
