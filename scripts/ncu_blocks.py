"""Per-basic-block instruction shares from an `ncu --page source --csv` (SASS) export.

Usage: python scripts/ncu_blocks.py SRC.csv [--per N] [--top 25] [--dump LO:HI]
--per N: divide execution counts by N (e.g. warp-neighbour evaluations) to read counts per unit.
"""
import argparse
import csv

ap = argparse.ArgumentParser()
ap.add_argument("src")
ap.add_argument("--per", type=float, default=1.0)
ap.add_argument("--top", type=int, default=25)
ap.add_argument("--dump", default="")
a = ap.parse_args()
rows = list(csv.reader(open(a.src)))
hdr = rows[1]
ia, isrc, ie = hdr.index("Address"), hdr.index("Source"), hdr.index("Instructions Executed")
iss = hdr.index("Warp Stall Sampling (All Samples)")
data = [(int(r[ia], 16), r[isrc], int(r[ie] or 0), int(r[iss] or 0)) for r in rows[2:] if len(r) > ie]
base = data[0][0]
tot = sum(d[2] for d in data)
print(f"total warp instructions {tot} ({tot / a.per:.1f} per unit)")
if a.dump:
    lo, hi = (int(x, 16) for x in a.dump.split(":"))
    for ad, s, e, smp in data:
        if lo <= ad - base <= hi:
            print(f"{ad - base:6x} {e / a.per:7.2f} {smp:7d}  {s}")
else:
    blocks, cur = [], None
    for ad, s, e, smp in data:
        if cur and e == cur[2]:
            cur[1] = ad; cur[3] += 1; cur[4] += smp
        else:
            if cur: blocks.append(cur)
            cur = [ad, ad, e, 1, smp]
    blocks.append(cur)
    blocks.sort(key=lambda b: -b[2] * b[3])
    for b in blocks[:a.top]:
        print(f"{b[0] - base:6x}-{b[1] - base:6x} per-unit {b[2] / a.per:6.2f} x {b[3]:3d} instr = {b[2] * b[3] / a.per:7.1f}"
              f"  share {b[2] * b[3] / tot:.3f}  stall-samples {b[4]}")
