for v in cur sp_base sp_o1 sp_sw sp_o1sw; do
  printf "%s " $v; LNS_LIB=build/variants/liblns_$v.so timeout 300 python scripts/probe_batch.py C4:49:400 C3:50:400 2>&1 | tail -2 | awk '{printf "%s %s  ", $1, $8}'; echo
  LNS_LIB=build/variants/liblns_$v.so timeout 300 python scripts/probe_single.py 2>&1 | tail -2 | tr '\n' ' '; echo
done
