# round-2 call S: where is the batched gap (cur vs split3): one phase of 49 x 3 CTAs, 148 x 1, 1 x 148
for v in cur split3 cur split3; do
  echo "== $v"
  LNS_LIB=build/variants/liblns_$v.so timeout 300 python scripts/probe_batch.py C4:49:400 C4:148:100 C4:1:400 C4:50:400 2>&1 | tail -4 | awk '{print $1, $2, $4, $5, $8}'
done
