# A/B of experimental builds (build/variants/liblns_<name>.so) on the bench job and one single search
for v in "$@"; do
  echo "== $v"
  LNS_LIB=build/variants/liblns_$v.so timeout 300 python scripts/probe_batch.py C4:50:400 C4:50:400 2>&1 | tail -1
  LNS_LIB=build/variants/liblns_$v.so timeout 300 python scripts/probe_batch.py C3:50:400 2>&1 | tail -1
done
