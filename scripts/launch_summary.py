"""Summarise an `ncu --metrics gpu__time_duration.sum --csv` launch list: launches, total us, share per kernel.

Usage: python scripts/launch_summary.py LAUNCHES.csv "header line" > profiles/..._summary.txt
"""
import csv
import sys
from collections import defaultdict

rows = [r for r in csv.reader(open(sys.argv[1])) if len(r) > 10]
hdr = rows[0]
ik, iv, iu = hdr.index("Kernel Name"), hdr.index("Metric Value"), hdr.index("Metric Unit")
tot, cnt = defaultdict(float), defaultdict(int)
scale = {"ns": 1e-3, "nsecond": 1e-3, "us": 1.0, "usecond": 1.0, "ms": 1e3, "msecond": 1e3, "s": 1e6, "second": 1e6}
for r in rows[1:]:
    if r[iu] not in scale:
        continue
    v = float(r[iv].replace(",", "")) * scale[r[iu]]
    tot[r[ik]] += v
    cnt[r[ik]] += 1
s = sum(tot.values())
print("# " + (sys.argv[2] if len(sys.argv) > 2 else "ncu launch list"))
print("# cold-cache, serialised per-launch times (gpu__time_duration.sum, --clock-control none); shares, not absolutes")
print("kernel | launches | total_us | share")
for k in sorted(tot, key=lambda k: -tot[k]):
    print(f"{k} | {cnt[k]} | {tot[k]:.1f} | {100 * tot[k] / s:.2f}%")
