"""Hot regions of an `ncu --page source --csv --print-source sass` export: per-instruction executed
counts (warp level) and stall samples, grouped into runs of consecutive instructions with the same
execution count (basic blocks). Usage: python scripts/sass_hot.py SASS.csv [units] [top]"""
import csv
import sys

rows = list(csv.reader(open(sys.argv[1])))
h = rows[1]
ia, isrc, ie, iss = h.index("Address"), h.index("Source"), h.index("Instructions Executed"), h.index("Warp Stall Sampling (All Samples)")
units = float(sys.argv[2]) if len(sys.argv) > 2 else 0.0
top = int(sys.argv[3]) if len(sys.argv) > 3 else 25
ins = []
for r in rows[2:]:
    if len(r) <= ie:
        continue
    ins.append((r[ia], r[isrc].strip(), int(r[ie] or 0), int(r[iss] or 0)))
tot = sum(x[2] for x in ins)
stall = sum(x[3] for x in ins)
blocks, cur = [], None
for i, x in enumerate(ins):
    if cur and x[2] == cur["count"]:
        cur["ins"].append(x)
    else:
        cur = {"count": x[2], "ins": [x], "start": i}
        blocks.append(cur)
for b in blocks:
    b["total"] = b["count"] * len(b["ins"])
    b["stall"] = sum(x[3] for x in b["ins"])
print(f"total warp instructions {tot:.4g}; per unit x32: {32 * tot / units:.1f}" if units else f"total {tot}")
for b in sorted(blocks, key=lambda b: -b["total"])[:top]:
    share = 100 * b["total"] / tot
    per = f" per-unit x32 {32 * b['total'] / units:.1f}" if units else ""
    print(f"--- block @{b['start']} len {len(b['ins'])} x {b['count']} = {share:.1f}% stall {100 * b['stall'] / max(stall, 1):.1f}%{per}")
    for x in b["ins"][:60]:
        print(f"   {x[3]:6d}  {x[1]}")
