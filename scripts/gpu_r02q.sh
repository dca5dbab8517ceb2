# round-2 call Q: interleaved repeated A/B (a fresh process per run) of cur vs split2 on the bench job
for rep in 1 2 3 4; do
  for v in cur split2; do
    printf "%s %s " $rep $v
    LNS_LIB=build/variants/liblns_$v.so timeout 300 python scripts/probe_batch.py C4:50:400 2>&1 | tail -1 | awk '{print $5, $8}'
  done
done
