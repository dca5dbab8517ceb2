"""Summarise an `ncu -i REP --page raw --csv` export of one kernel launch into profiles/*.json.

Usage: python scripts/ncu_summary.py RAW.csv OUT.json --kernel "..." --capture "..."
Keeps the metrics the roofline / pipe analysis in DESIGN.md cites; dram bytes per launch =
dram__bytes_read.sum + dram__bytes_write.sum (the bench's roofline "traffic").
"""
import argparse
import csv
import json

KEEP = [
    "gpu__time_duration.sum", "smsp__issue_active.avg.pct_of_peak_sustained_active",
    "sm__inst_executed_pipe_alu.avg.pct_of_peak_sustained_active",
    "sm__inst_executed_pipe_fma.avg.pct_of_peak_sustained_active",
    "sm__inst_executed_pipe_fmaheavy.avg.pct_of_peak_sustained_active",
    "sm__inst_executed_pipe_xu.avg.pct_of_peak_sustained_active",
    "sm__inst_executed_pipe_lsu.avg.pct_of_peak_sustained_active",
    "sm__inst_executed_pipe_adu.avg.pct_of_peak_sustained_active",
    "sm__inst_executed_pipe_uniform.avg.pct_of_peak_sustained_active",
    "l1tex__data_pipe_lsu_wavefronts_mem_shared.sum.pct_of_peak_sustained_elapsed",
    "l1tex__data_bank_conflicts_pipe_lsu_mem_shared.sum",
    "sm__warps_active.avg.pct_of_peak_sustained_active", "launch__registers_per_thread",
    "launch__grid_size", "launch__block_size", "smsp__inst_executed.sum",
    "sm__cycles_elapsed.avg.per_second", "dram__bytes_read.sum", "dram__bytes_write.sum",
    "smsp__warps_eligible.avg.per_cycle_active",
    "smsp__average_warp_latency_issue_stalled_barrier.ratio",
    "smsp__average_warp_latency_issue_stalled_short_scoreboard.ratio",
    "smsp__average_warp_latency_issue_stalled_math_pipe_throttle.ratio",
    "smsp__average_warp_latency_issue_stalled_wait.ratio",
    "smsp__average_warp_latency_issue_stalled_not_selected.ratio",
    "smsp__average_warp_latency_issue_stalled_selected.ratio",
]
SCALE = {"byte": 1, "Kbyte": 1e3, "Mbyte": 1e6, "Gbyte": 1e9}


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("raw")
    ap.add_argument("out")
    ap.add_argument("--kernel", required=True)
    ap.add_argument("--capture", required=True)
    ap.add_argument("--source", help="`--page source --csv` export of the same capture (per-SASS counts)")
    ap.add_argument("--units", type=float, default=0.0, help="neighbour evaluations in the profiled launch")
    ap.add_argument("--source-sha", default=None, help="_build.source_hash() of the profiled build")
    a = ap.parse_args()
    with open(a.raw) as fh:
        rows = list(csv.reader(fh))
    hdr, units = rows[0], rows[1]
    data = rows[2]  # the first (profiled) launch
    metrics = {}
    for name, unit, val in zip(hdr, units, data):
        if name in KEEP or ("pipe_" in name and name.endswith(".avg.pct_of_peak_sustained_active")) or \
                (name.startswith("smsp__average_warps_issue_stalled_") and name.endswith("_per_issue_active.ratio")):
            metrics[name] = [val, unit]

    def nbytes(key):
        v, u = metrics.get(key, ["0", "byte"])
        return float(v.replace(",", "")) * SCALE.get(u, 1)

    out = {"kernel": a.kernel, "capture": a.capture, "source_sha": a.source_sha,
           "dram_bytes_per_launch": nbytes("dram__bytes_read.sum") + nbytes("dram__bytes_write.sum"),
           "metrics": metrics}
    if a.source and a.units:
        src = list(csv.reader(open(a.source)))
        h = src[1]
        isrc, ie = h.index("Source"), h.index("Instructions Executed")
        tot = popc = 0
        mix = {}
        for r in src[2:]:
            if len(r) <= ie:
                continue
            e = int(r[ie] or 0)
            tot += e
            op = r[isrc].split()
            op = op[1] if op and op[0].startswith("@") and len(op) > 1 else (op[0] if op else "")
            op = op.split(".")[0]
            mix[op] = mix.get(op, 0) + e
            if op == "POPC":
                popc += e
        # warp-level counts x 32 lanes / neighbours = per-neighbour (per-lane) instruction counts
        out["per_neighbor"] = {"units": a.units, "issued_instructions": 32 * tot / a.units,
                               "popc": 32 * popc / a.units,
                               "mix": {k: round(32 * v / a.units, 2) for k, v in
                                       sorted(mix.items(), key=lambda kv: -kv[1])[:16]}}
    stalls = {k.replace("smsp__average_warps_issue_stalled_", "").replace("_per_issue_active.ratio", ""):
              float(v[0].replace(",", "")) for k, v in metrics.items()
              if k.startswith("smsp__average_warps_issue_stalled_") and k.endswith("_per_issue_active.ratio")}
    out["stalls_per_issue"] = dict(sorted(stalls.items(), key=lambda kv: -kv[1]))
    with open(a.out, "w") as fh:
        json.dump(out, fh, indent=1)
    print(json.dumps(out, indent=1)[:3000])


if __name__ == "__main__":
    main()
