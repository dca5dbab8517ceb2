for v in cur split3 cur split3; do
  echo "== $v"; LNS_LIB=build/variants/liblns_$v.so timeout 300 python scripts/probe_clocks.py 2>&1 | tail -1
done
