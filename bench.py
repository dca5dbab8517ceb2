#!/usr/bin/env python
"""Benchmark of the B200 k-Hamming tabu search.

Contract: ``python bench.py --gpus N --steps K --warmup W [--impl reference]`` prints ONE JSON
line on rank 0.

Workload (BASELINE.json ``metric`` "PPP 3-Hamming neighbors evaluated/sec and tabu iters/sec at
1/2/4/8 B200", quoted at 1/2/4/8 GPUs on configs[3]): the planted PPP instance m = 101, n = 117
(seed 1004), 3-Hamming neighbourhood (C(117,3) = 260,130 neighbours per iteration), tabu tenure
floor(M/6) = 43,355, run the way the paper runs it: "A tabu search was executed 50 times"
(Table III). One STEP = the 50 independent searches of 400 iterations each (the
paper's cap C(n,3) = 260,130 iterations is scaled down; no early stop), run r of step s starting
from splitmix64(seed_s + r). Every iteration of every search evaluates all 260,130 neighbours,
selects the best admissible one and moves. On each GPU the searches run batched in one
persistent kernel (the grid split into groups, ``lns_tabu_run_batch``); with N GPUs run r goes
to rank r mod N (no per-iteration collective; the total job is fixed -> strong scaling).

``value`` = neighbours evaluated per second over the whole job (device time by CUDA events, max
over ranks), inputs resident in HBM. ``e2e`` = the same job through the C ABI with HOST buffers
(instance upload, start vectors, final vectors and results back inside the timed region).
``single_search`` = one search at a time (latency view: all SMs on one search, 2,000 iterations).
``c5_single_search`` = BASELINE configs[4] (1024 x 1024, 3-Hamming), one search, 5 iterations.
``ubqp_single_search`` = the second binary fitness (UBQP): k = 3, n = 500, one
search, 50 iterations (context; not part of the headline).
``c5_restarts`` = BASELINE configs[4]'s restart job per GPU: 8 restarts of C5 per GPU (64 on 8
GPUs), a few iterations each, through lns_tabu_run_batch (sharded by the library over the NCCL
communicator when N > 1).
``partitioned`` = ONE search whose neighbourhood is partitioned over the N GPUs:
C4 (2,000 iterations) and C5 (5 iterations) with one NCCL u64-MIN all-reduce per iteration
(lns_attach_comm on torch's communicator), and the device-initiated exchange (peer_tabu_run, C4).
At N = 1 it is the single-GPU persistent search.
``roofline`` = the search kernel's issued integer instructions against the MEASURED issue peak
(profiles/int_peaks.json), with the binding pipe (POPC on XU) against its measured peak; the
per-neighbour instruction counts come from the committed ncu capture, which must have been taken
from the current sources (hash check; a stale capture aborts the bench).
``cpu_baseline`` = the CPU oracle on this host on a bounded sample, all cores and single-threaded.
``--impl reference`` times that oracle alone as the reference arm (this paper has no code).

``--gpus N`` with N > 1 and no torchrun environment re-launches this script under
``torch.distributed.run`` with N ranks (127.0.0.1); with fewer than N visible GPUs it fails.
"""
from __future__ import annotations

import argparse
import json
import os
import statistics
import subprocess
import sys
import tempfile
import threading
import time
from math import comb

ROOT = os.path.dirname(os.path.abspath(__file__))
sys.path.insert(0, ROOT)

import numpy as np  # noqa: E402

import ppp_inputs as pi  # noqa: E402

METRIC = "PPP 3-Hamming neighbors evaluated/sec and tabu iters/sec at 1/2/4/8 B200"
UNIT = "neighbors/s"
CFG = "C4"
RUNS = 50        # independent searches per step
ITERS = 400      # iterations per search per step
SINGLE_ITERS = 2000
C5_ITERS = 5     # C5 iterations timed beside the headline (9.5 ms each)
C5_RESTARTS_PER_GPU = 8  # BASELINE configs[4]: 64 restarts sharded across 8 x B200
C5_RESTART_ITERS = 3
PART_C4_ITERS = 2000
PART_C5_ITERS = 5
L2_FLUSH_BYTES = 512 << 20  # > 126 MB L2
CONTEXT_BUDGET_S = float(os.environ.get("LNS_BENCH_CONTEXT_BUDGET_S", "300"))  # watchdog of the context lines
PROFILE = os.path.join(ROOT, "profiles", "ncu_k_search_bench.json")  # ncu --set full of one bench step
INT_PEAKS = os.path.join(ROOT, "profiles", "int_peaks.json")  # scripts/int_peaks.cu on the B200


def env_int(name, default):
    try:
        return int(os.environ.get(name, default))
    except ValueError:
        return default


def peaks():
    try:
        with open(os.path.join(ROOT, "MEASURED_PEAKS.json")) as fh:
            return json.load(fh), "measured"
    except OSError:
        return {"sm_max_mhz": 1965.0, "hbm_gbs": 6650.0}, "fallback"


class ContextLines:
    """The JSON line's context sections after the headline. section(name, fn) stores fn() in
    line[name], or {"error": ...} if it raises; a watchdog prints the line (rank 0) and ends the
    process with status 0 if finish() has not been called after `budget` seconds, so a context
    collective that some rank never reaches cannot hold back the measured headline."""

    def __init__(self, line: dict, rank: int, budget: float):
        self.line, self.rank, self.budget = line, rank, budget
        self.emitted, self.done = False, threading.Event()
        threading.Thread(target=self._watchdog, daemon=True).start()

    def emit(self, note=None):
        if self.rank == 0 and not self.emitted:
            self.emitted = True
            if note:
                self.line["context_note"] = note
            print(json.dumps(self.line), flush=True)

    def _watchdog(self):
        if not self.done.wait(self.budget):
            self.emit(f"context lines stopped after {self.budget:.0f} s (a context section did not finish on every "
                      "rank); the headline, e2e and roofline above are complete")
            os._exit(0)

    def section(self, name, fn):
        try:
            self.line[name] = fn()
        except Exception as e:  # noqa: BLE001 -- a context line must not take the headline down
            self.line[name] = {"error": f"{type(e).__name__}: {e}"[:400]}
            print(f"[bench] {name} failed: {e}", file=sys.stderr)

    def finish(self):
        self.done.set()
        self.emit()


def run_seed(step: int) -> int:
    return 5 + step


class ClockSampler:
    """nvidia-smi clocks and throttle reasons sampled every 50 ms during the timed region."""

    FIELDS = ["clocks.sm", "clocks.max.sm", "power.draw", "clocks_event_reasons.hw_slowdown",
              "clocks_event_reasons.hw_thermal_slowdown", "clocks_event_reasons.sw_thermal_slowdown",
              "clocks_event_reasons.sw_power_cap"]

    def __init__(self, gpu_index: int):
        self.gpu = gpu_index
        self.proc = None
        self.path = None

    def __enter__(self):
        fd, self.path = tempfile.mkstemp(suffix=".csv")
        os.close(fd)
        try:
            self.proc = subprocess.Popen(
                ["nvidia-smi", f"--query-gpu={','.join(self.FIELDS)}", "--format=csv,noheader,nounits",
                 "-lms", "50", "-i", str(self.gpu)], stdout=open(self.path, "w"), stderr=subprocess.DEVNULL)
        except OSError:
            self.proc = None
        time.sleep(0.3)
        return self

    def __exit__(self, *exc):
        if self.proc is not None:
            self.proc.terminate()
            try:
                self.proc.wait(timeout=5)
            except subprocess.TimeoutExpired:
                self.proc.kill()

    def summary(self):
        rows = []
        try:
            with open(self.path) as fh:
                for line in fh:
                    p = [x.strip() for x in line.split(",")]
                    if len(p) == len(self.FIELDS):
                        rows.append(p)
        except OSError:
            pass
        finally:
            try:
                os.unlink(self.path)
            except OSError:
                pass
        if not rows:
            return {"sm_mhz": None, "sm_max_mhz": None, "reasons": ["unavailable"], "samples": 0}
        sm = [float(r[0]) for r in rows if r[0].replace(".", "").isdigit()]
        loaded = [x for x in sm if x > 600] or sm
        names = ["hw_slowdown", "hw_thermal_slowdown", "sw_thermal_slowdown", "sw_power_cap"]
        reasons = sorted({names[i] for r in rows for i in range(4) if r[3 + i].lower().startswith("active")})
        pw = [float(r[2]) for r in rows if r[2].replace(".", "").isdigit()]
        return {"sm_mhz": statistics.median(loaded) if loaded else None,
                "sm_max_mhz": float(rows[0][1]) if rows[0][1].replace(".", "").isdigit() else None,
                "reasons": reasons, "samples": len(rows), "power_w_max": max(pw) if pw else None}


def start_vectors(n: int, step: int, runs) -> np.ndarray:
    runs = list(runs)
    if not runs:
        return np.zeros((0, n), np.int8)
    return np.stack([pi.start_vector(n, pi.restart_seed(run_seed(step), r)) for r in runs]).astype(np.int8)


# --------------------------------------------------------------------------------- oracle arm
def oracle_sample(budget_s: float, nthreads: int = 0, per_run: int = ITERS):
    """The CPU oracle (as it stands) on the same job: the first `per_run` iterations of runs 0, 1,
    ... of step 0, as many runs as fit ~budget_s. Returns (neighbors/s, iters/s, iterations,
    runs, cores, seconds)."""
    import oracle

    c = pi.CONFIGS[CFG]
    inst = pi.config_instance(CFG)
    M = comb(inst.n, c["k"])
    ten = pi.default_tenure(inst.n, c["k"])
    iters, runs, t = 0, 0, time.perf_counter()
    while True:
        V0 = start_vectors(inst.n, 0, [runs])[0]
        oracle.tabu_run(inst.A, inst.S, c["k"], V0, per_run, ten, stop_on_zero=False, nthreads=nthreads)
        iters += per_run
        runs += 1
        if time.perf_counter() - t >= budget_s or runs >= RUNS:
            break
    dt = time.perf_counter() - t
    cores = nthreads or oracle.max_threads()
    return iters * M / dt, iters / dt, iters, runs, cores, dt


def cpu_model() -> str:
    try:
        with open("/proc/cpuinfo") as fh:
            for line in fh:
                if line.startswith("model name"):
                    return line.split(":", 1)[1].strip()
    except OSError:
        pass
    return "unknown"


def relaunch_under_torchrun(args) -> int:
    """--gpus N (N > 1) without a torchrun environment: start N ranks on this node ourselves."""
    import torch

    have = torch.cuda.device_count()
    if have < args.gpus:
        print(json.dumps({"error": f"bench.py --gpus {args.gpus} needs {args.gpus} visible GPUs, found {have}"}),
              flush=True)
        return 2
    cmd = [sys.executable, "-m", "torch.distributed.run", "--nnodes=1", f"--nproc-per-node={args.gpus}",
           "--master-addr=127.0.0.1", f"--master-port={29400 + os.getpid() % 1000}", os.path.abspath(__file__),
           *sys.argv[1:]]
    return subprocess.call(cmd)


def run_reference(args, rank, world):
    """--impl reference: the CPU oracle (this paper has no code). Each step = the
    first 2 runs of the job, 4 iterations each (a bounded sample of the same workload)."""
    if rank != 0:
        return
    import oracle

    oracle.build()
    c = pi.CONFIGS[CFG]
    inst = pi.config_instance(CFG)
    M = comb(inst.n, c["k"])
    ten = pi.default_tenure(inst.n, c["k"])
    runs, per_run = 2, 4
    times = []
    for s in range(args.warmup + args.steps):
        V0 = start_vectors(inst.n, s, range(runs))
        t = time.perf_counter()
        for r in range(runs):
            oracle.tabu_run(inst.A, inst.S, c["k"], V0[r], per_run, ten, stop_on_zero=False)
        if s >= args.warmup:
            times.append(time.perf_counter() - t)
    total = sum(times)
    value = args.steps * runs * per_run * M / total
    cores = oracle.max_threads()
    sample = f"{runs} runs x {per_run} tabu iterations of {CFG} per step, from-scratch fitness ({cores} OpenMP threads)"
    line = {
        "impl": "reference", "metric": METRIC, "value": value, "unit": UNIT, "n_gpus": args.gpus,
        "steps": args.steps, "warmup": args.warmup, "ms_per_step": 1e3 * total / args.steps,
        "higher_is_better": True, "scaling": "strong", "vs_baseline": None, "dtype": "int32",
        "data": "synthetic planted PPP instance (seeded splitmix64)",
        "config": {"workload": f"{CFG}: PPP m=101 n=117, 3-Hamming, tenure {ten}, independent tabu searches",
                   "runs_per_step": runs, "iters_per_run": per_run, "parallelism": "cpu-openmp",
                   "l2": "n/a (CPU)"},
        "tabu_iters_per_s": args.steps * runs * per_run / total,
        "cpu_baseline": {"value": value, "unit": UNIT, "cores": cores, "kind": "oracle", "sample": sample},
        "e2e": {"value": value, "unit": UNIT, "h2d_bytes_per_step": 0, "d2h_bytes_per_step": 0},
    }
    print(json.dumps(line), flush=True)


# --------------------------------------------------------------------------------- GPU arm
def timed(stream, fn):
    """Device time (ms) of fn() on `stream` by CUDA events, synchronised on both sides."""
    import torch

    torch.cuda.synchronize()
    a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    a.record(stream)
    out = fn()
    b.record(stream)
    torch.cuda.synchronize()
    return a.elapsed_time(b), out


def max_over_ranks(vals, world, dev):
    """Element-wise max of a list of floats over ranks (device timing: the slowest rank)."""
    if world == 1:
        return list(vals)
    import torch
    import torch.distributed as dist

    t = torch.tensor(vals, dtype=torch.float64, device=dev)
    dist.all_reduce(t, op=dist.ReduceOp.MAX)
    return [float(x) for x in t]


def sum_over_ranks(vals, world, dev):
    if world == 1:
        return list(vals)
    import torch
    import torch.distributed as dist

    t = torch.tensor(vals, dtype=torch.int64, device=dev)
    dist.all_reduce(t, op=dist.ReduceOp.SUM)
    return [int(x) for x in t]


def roofline_of(nbr_per_s_kernel, sms):
    """The search kernel against the MEASURED integer peaks. The per-neighbour
    instruction counts come from the committed ncu capture of the same kernel and job; a capture
    taken from other sources than the current ones is refused (it would be silently stale)."""
    from paper_conf_ipps_luongmt10_b200 import _build

    pk, src = peaks()
    mhz = float(pk.get("sm_max_mhz", 1965.0))
    if not os.path.exists(PROFILE):
        raise SystemExit(f"bench.py: {PROFILE} missing (capture it with scripts/capture_bench_kernel.sh)")
    with open(PROFILE) as fh:
        prof = json.load(fh)
    want = _build.source_hash()
    if prof.get("source_sha") != want:
        raise SystemExit(f"bench.py: the committed ncu capture {os.path.relpath(PROFILE, ROOT)} was taken from "
                         f"sources {prof.get('source_sha')}, the current sources are {want}: re-capture it "
                         "(scripts/capture_bench_kernel.sh) instead of reporting stale per-neighbour counts")
    per = prof["per_neighbor"]
    ipn, ppn = per["issued_instructions"], per["popc"]
    if os.path.exists(INT_PEAKS):
        with open(INT_PEAKS) as fh:
            ip = json.load(fh)
        issue_lanes = ip["peaks"]["mix_lop3_imad"]["lanes_per_clk_per_sm"]
        popc_lanes = ip["peaks"]["popc"]["lanes_per_clk_per_sm"]
        peak_src = (f"measured on B200 (profiles/int_peaks.json: LOP3/IMAD alternating {issue_lanes:.1f}, "
                    f"POPC {popc_lanes:.1f} lanes/clk/SM) x {sms} SMs x {mhz:.0f} MHz ({src} sm_max_mhz)")
    else:
        issue_lanes, popc_lanes = 128.0, 16.0
        peak_src = f"fallback 128 / 16 lanes/clk/SM (no profiles/int_peaks.json) x {sms} SMs x {mhz:.0f} MHz"
    peak = sms * issue_lanes * mhz * 1e6 / 1e12
    achieved = nbr_per_s_kernel * ipn / 1e12
    xu_ceiling = sms * popc_lanes * mhz * 1e6 / ppn
    m, k = pi.CONFIGS[CFG]["m"], pi.CONFIGS[CFG]["k"]
    ops = m * (k + 4)
    return {"bound": "alu", "achieved": achieved, "peak": peak, "unit": "Tops/s", "frac": achieved / peak,
            "traffic": prof.get("dram_bytes_per_launch"),
            "kernel": "k_search<3> (persistent, batched searches)",
            "achieved_is": "issued thread-instructions/s = live neighbours/s (CUDA events) x issued instructions "
                           "per neighbour (ncu source page of the committed capture, same sources)",
            "instructions_per_neighbor": ipn, "peak_source": peak_src, "capture_source_sha": want,
            "binding_pipe": {"pipe": "xu (POPC)", "popc_per_neighbor": ppn,
                             "peak_lanes_per_clk_per_sm": popc_lanes,
                             "ceiling_neighbors_per_s": xu_ceiling, "frac": nbr_per_s_kernel / xu_ceiling},
            "stalls_per_issue": prof.get("stalls_per_issue"),
            "model": {"ops_per_neighbor": ops, "frac": nbr_per_s_kernel * ops / 1e12 / peak,
                      "note": "SURVEY.md §8(d) m(k+4) model; the bit-sliced kernel needs fewer ops, so > 1 is possible"}}


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--gpus", type=int, default=1)
    ap.add_argument("--steps", type=int, default=5)
    ap.add_argument("--warmup", type=int, default=3)
    ap.add_argument("--impl", default="lns", choices=["lns", "reference"])
    ap.add_argument("--iters", type=int, default=ITERS)
    ap.add_argument("--runs", type=int, default=RUNS)
    ap.add_argument("--no-cpu-baseline", action="store_true")
    ap.add_argument("--no-single", action="store_true")
    ap.add_argument("--no-c5", action="store_true")
    ap.add_argument("--no-ubqp", action="store_true")
    ap.add_argument("--no-partitioned", action="store_true")
    ap.add_argument("--cpu-budget", type=float, default=10.0)
    args = ap.parse_args()
    in_torchrun = "WORLD_SIZE" in os.environ
    rank, world, local = env_int("RANK", 0), env_int("WORLD_SIZE", 1), env_int("LOCAL_RANK", 0)
    if args.impl == "reference":  # the CPU oracle: rank 0 alone works, other ranks exit 0
        run_reference(args, rank, world)
        return
    if args.gpus > 1 and not in_torchrun:
        sys.exit(relaunch_under_torchrun(args))
    if world != args.gpus:
        print(json.dumps({"error": f"bench.py --gpus {args.gpus} launched with WORLD_SIZE={world}"}), flush=True)
        sys.exit(2)
    args.warmup = max(args.warmup, 3)

    import torch
    import torch.distributed as dist

    import paper_conf_ipps_luongmt10_b200 as L
    from paper_conf_ipps_luongmt10_b200 import parallel as par

    torch.cuda.set_device(local)
    dev = torch.device("cuda", local)
    if world > 1:
        dist.init_process_group("nccl", device_id=dev)
    c = pi.CONFIGS[CFG]
    k = c["k"]
    inst = pi.config_instance(CFG)
    M = comb(inst.n, k)
    ten = pi.default_tenure(inst.n, k)
    iters = args.iters
    mine = par.restart_shard(args.runs, rank, world)  # runs of this rank: r = rank, rank + world, ...
    R = len(mine)
    ctx = L.lns_create(inst.A, inst.S, local)
    stream = torch.cuda.current_stream(dev)
    nsteps = args.warmup + args.steps
    V0s = [torch.from_numpy(start_vectors(inst.n, s, mine)).to(dev) for s in range(nsteps)]
    Vo = torch.empty((max(R, 1), inst.n), dtype=torch.int8, device=dev)
    flush = torch.empty(L2_FLUSH_BYTES // 4, dtype=torch.int32, device=dev)

    def barrier():
        if world > 1:
            dist.barrier()

    def step(s):
        if R == 0:
            return []
        return L.lns_tabu_run_batch(ctx, k, R, iters, ten, 0, V0s[s], 0, Vo, stream)

    # ---- headline: the C4 job, inputs resident in HBM
    for s in range(args.warmup):
        step(s)
    torch.cuda.synchronize()
    ev0 = [torch.cuda.Event(enable_timing=True) for _ in range(args.steps)]
    ev1 = [torch.cuda.Event(enable_timing=True) for _ in range(args.steps)]
    kernel_ms, iters_done = [], 0
    with ClockSampler(local) as clk:
        for i in range(args.steps):
            flush.fill_(i)  # evict L2 between timed steps
            barrier()
            torch.cuda.synchronize()
            ev0[i].record(stream)
            res = step(args.warmup + i)
            ev1[i].record(stream)
            torch.cuda.synchronize()
            kernel_ms.append(L.lns_last_kernel_ms(ctx) if R else 0.0)
            iters_done += sum(r["iters_done"] for r in res)
    clocks = clk.summary()
    step_ms = [a.elapsed_time(b) for a, b in zip(ev0, ev1)]
    my_iters = iters_done
    total_ms, kern_ms = max_over_ranks([sum(step_ms), sum(kernel_ms)], world, dev)
    (iters_done,) = sum_over_ranks([iters_done], world, dev)
    value = iters_done * M / (total_ms / 1e3)

    # ---- end to end through the C ABI with host buffers (pinned), same job
    A_h = torch.from_numpy(inst.A).pin_memory()
    S_h = torch.from_numpy(inst.S).pin_memory()
    V0_h = [torch.from_numpy(start_vectors(inst.n, s, mine)).pin_memory() for s in range(nsteps)]
    Vo_h = torch.empty((max(R, 1), inst.n), dtype=torch.int8).pin_memory()
    for s in range(args.warmup):  # untimed, like the device leg (first-context costs land here)
        c2 = L.lns_create(A_h, S_h, local)
        if R:
            L.lns_tabu_run_batch(c2, k, R, iters, ten, 0, V0_h[s], 0, Vo_h, stream)
        L.lns_destroy(c2)
    torch.cuda.synchronize()
    e2e_ms, e2e_iters, e2e_steps = 0.0, 0, []
    for i in range(args.steps):
        flush.fill_(i)
        barrier()

        def e2e_step():
            c2 = L.lns_create(A_h, S_h, local)
            r2 = L.lns_tabu_run_batch(c2, k, R, iters, ten, 0, V0_h[args.warmup + i], 0, Vo_h, stream) if R else []
            L.lns_destroy(c2)
            return r2

        ms, r2 = timed(stream, e2e_step)
        e2e_steps.append(ms)
        e2e_ms += ms
        e2e_iters += sum(r["iters_done"] for r in r2)
    (e2e_ms,) = max_over_ranks([e2e_ms], world, dev)
    (e2e_iters,) = sum_over_ranks([e2e_iters], world, dev)
    e2e_value = e2e_iters * M / (e2e_ms / 1e3)
    if rank == 0:
        print(f"[bench] e2e ms per step: {[round(x, 2) for x in e2e_steps]}", file=sys.stderr)
    h2d = A_h.numel() + 4 * S_h.numel() + V0_h[0].numel()
    d2h = Vo_h.numel() + 48 * R  # final vectors + lns_result records

    # ---- the headline line; the context lines below fill it in. Each context section is guarded:
    #      an exception becomes {"error": ...} in its slot, and a watchdog prints the line and ends the
    #      process if the sections have not finished after CONTEXT_BUDGET_S (a collective of a context
    #      line that one rank never reaches cannot hold back the measured headline).
    sms = torch.cuda.get_device_properties(dev).multi_processor_count
    kern_avg_s = kern_ms / 1e3 / args.steps
    nbr_per_s_kernel = (my_iters / args.steps) * M / kern_avg_s if kern_avg_s > 0 else 0.0
    roofline = roofline_of(nbr_per_s_kernel, sms)
    line = {
        "metric": METRIC, "value": value, "unit": UNIT, "n_gpus": world, "steps": args.steps,
        "warmup": args.warmup, "ms_per_step": total_ms / args.steps, "higher_is_better": True,
        "scaling": "strong", "vs_baseline": None, "dtype": "int32",
        "data": "synthetic planted PPP instance (seeded splitmix64, DESIGN.md §3)",
        "config": {"workload": f"{CFG}: PPP m=101 n=117, 3-Hamming (260,130 neighbours/iteration), tenure {ten}; "
                               f"{args.runs} independent tabu searches x {iters} iterations per step "
                               "(PAPER.md:250 protocol), no early stop",
                   "runs_per_step": args.runs, "iters_per_run": iters,
                   "parallelism": f"runs sharded over {world} GPUs (r mod N), batched per GPU" if world > 1
                   else "1 GPU, runs batched in one persistent kernel",
                   "l2": "flushed (512 MiB write) between timed steps"},
        "tabu_iters_per_s": iters_done / (total_ms / 1e3),
        "e2e": {"value": e2e_value, "unit": UNIT, "h2d_bytes_per_step": h2d, "d2h_bytes_per_step": d2h,
                "tabu_iters_per_s": e2e_iters / (e2e_ms / 1e3)},
        "single_search": None, "partitioned": None, "c5_single_search": None, "c5_restarts": None,
        "ubqp_single_search": None, "ubqp_restarts": None,
        # our kernels per timed step: k_init_slots + the persistent k_search
        "gpu_launches": args.steps * 2,
        "clocks": clocks,
        "roofline": roofline,
        "cpu_baseline": None,
    }
    ctxl = ContextLines(line, rank, CONTEXT_BUDGET_S)
    section = ctxl.section

    # ---- single search (latency view), N = 1 only
    def single_search():
        tr = torch.empty(SINGLE_ITERS, dtype=torch.int64, device=dev)
        tf = torch.empty(SINGLE_ITERS, dtype=torch.int64, device=dev)
        v1 = torch.empty(inst.n, dtype=torch.int8, device=dev)
        v0 = V0s[0][0].contiguous()
        L.lns_tabu_run(ctx, k, SINGLE_ITERS, ten, 0, v0, 0, v1, tr, tf, stream)
        ms = []
        for _ in range(3):
            flush.fill_(0)
            ms.append(timed(stream, lambda: L.lns_tabu_run(ctx, k, SINGLE_ITERS, ten, 0, v0, 0, v1, tr, tf, stream))[0])
        best = min(ms)
        return {"neighbors_per_s": SINGLE_ITERS * M / (best / 1e3), "tabu_iters_per_s": SINGLE_ITERS / (best / 1e3),
                "us_per_iteration": 1e3 * best / SINGLE_ITERS, "iters": SINGLE_ITERS,
                "note": "one search on all SMs (persistent kernel, one exchange per iteration)"}

    if world == 1 and not args.no_single:
        section("single_search", single_search)

    # ---- C5 (BASELINE configs[4], 1024 x 1024, 3-Hamming, 1.78e8 neighbours per iteration): one
    #      search on all SMs, a few iterations (N = 1 only; context beside the headline)
    inst5 = pi.config_instance("C5")
    M5 = comb(inst5.n, 3)

    def c5_single():
        with L.Instance(inst5.A, inst5.S) as I5:
            L.lns_tabu_run(I5.ctx, 3, 1, -1, pi.config_seed("C5"), None, 0)
            ms5 = []
            for _ in range(2):
                flush.fill_(0)
                torch.cuda.synchronize()
                L.lns_tabu_run(I5.ctx, 3, C5_ITERS, -1, pi.config_seed("C5"), None, 0)
                ms5.append(L.lns_last_kernel_ms(I5.ctx))
        b5 = min(ms5)
        return {"neighbors_per_s": C5_ITERS * M5 / (b5 / 1e3), "tabu_iters_per_s": C5_ITERS / (b5 / 1e3),
                "ms_per_iteration": b5 / C5_ITERS, "iters": C5_ITERS,
                "note": "C5 single search from the config seed (packed plan for m > 255, DESIGN.md §5.11); device time of the launch"}

    if world == 1 and not args.no_c5:
        section("c5_single_search", c5_single)

    # ---- C5 restarts (BASELINE configs[4]: "64 independent restarts sharded across 8 x B200"):
    #      8 restarts per GPU through lns_tabu_run_batch; with N > 1 the library shards restart r
    #      to rank r mod N over the attached NCCL communicator and gathers every result
    def c5_restarts():
        R5 = C5_RESTARTS_PER_GPU * world
        with L.Instance(inst5.A, inst5.S, local) as I5:
            comm = par.nccl_comm_ptr(device=dev) if world > 1 else None
            if comm:
                L.lns_attach_comm(I5.ctx, comm, rank, world)
            L.lns_tabu_run_batch(I5.ctx, 3, R5, 1, -1, 1005, None, 0)  # warm-up (buffers)
            barrier()
            ms, r5 = timed(stream, lambda: L.lns_tabu_run_batch(I5.ctx, 3, R5, C5_RESTART_ITERS, -1, 1005, None, 0))
            kms = L.lns_last_kernel_ms(I5.ctx)
            if comm:
                L.lns_attach_comm(I5.ctx, None, 0, 1)
        ms, kms = max_over_ranks([ms, kms], world, dev)
        done5 = sum(r["iters_done"] for r in r5)  # every rank holds every restart's result
        return {"restarts": R5, "restarts_per_gpu": C5_RESTARTS_PER_GPU, "iters_per_restart": C5_RESTART_ITERS,
                "neighbors_per_s": done5 * M5 / (ms / 1e3), "tabu_iters_per_s": done5 / (ms / 1e3),
                "kernel_neighbors_per_s": done5 * M5 / (kms / 1e3) if kms > 0 else None,
                "note": "lns_tabu_run_batch, restart r on rank r mod N, results gathered by the library (NCCL)"}

    if not args.no_c5:
        section("c5_restarts", c5_restarts)

    # ---- one search partitioned over the N GPUs
    def partitioned():
        part = {}
        comm = par.nccl_comm_ptr(device=dev) if world > 1 else None
        for name, inst_p, kp, itp in (("C4", inst, 3, PART_C4_ITERS), ("C5", inst5, 3, PART_C5_ITERS)):
            Mp = comb(inst_p.n, kp)
            with L.Instance(inst_p.A, inst_p.S, local) as Ip:
                if comm:
                    L.lns_attach_comm(Ip.ctx, comm, rank, world)
                trp = torch.empty(itp, dtype=torch.int64, device=dev)
                v0 = torch.from_numpy(pi.start_vector(inst_p.n, pi.config_seed(name))).to(dev)
                L.lns_tabu_run(Ip.ctx, kp, min(itp, 70), -1, 0, v0, 0, None, trp, None, stream)  # warm-up
                barrier()
                ms, _ = timed(stream, lambda: L.lns_tabu_run(Ip.ctx, kp, itp, -1, 0, v0, 0, None, trp, None, stream))
                trace_sha = __import__("hashlib").sha256(trp.cpu().numpy().tobytes()).hexdigest()[:16]
                if comm:
                    L.lns_attach_comm(Ip.ctx, None, 0, 1)
            (ms,) = max_over_ranks([ms], world, dev)
            part[name] = {"iters": itp, "us_per_iteration": 1e3 * ms / itp, "tabu_iters_per_s": itp / (ms / 1e3),
                          "neighbors_per_s": itp * Mp / (ms / 1e3), "trace_sha16": trace_sha,
                          "exchange": "ncclAllReduce u64 MIN per iteration (lns_attach_comm, CUDA-graph stepped loop)"
                          if world > 1 else "none (N = 1: the persistent single-GPU search)"}
        if world > 1:  # the device-initiated exchange: persistent kernels meet in peer memory
            with L.Instance(inst.A, inst.S, local) as Ip:
                trp = torch.empty(PART_C4_ITERS, dtype=torch.int64, device=dev)
                v0 = torch.from_numpy(pi.start_vector(inst.n, pi.config_seed("C4"))).to(dev)
                par.peer_tabu_run(Ip.ctx, 3, 70, -1, 0, v0, 0, trace_rank=trp, stream=stream)
                barrier()
                ms, _ = timed(stream, lambda: par.peer_tabu_run(Ip.ctx, 3, PART_C4_ITERS, -1, 0, v0, 0,
                                                                trace_rank=trp, stream=stream))
                trace_sha = __import__("hashlib").sha256(trp.cpu().numpy().tobytes()).hexdigest()[:16]
            (ms,) = max_over_ranks([ms], world, dev)
            part["C4_peer"] = {"iters": PART_C4_ITERS, "us_per_iteration": 1e3 * ms / PART_C4_ITERS,
                               "tabu_iters_per_s": PART_C4_ITERS / (ms / 1e3),
                               "neighbors_per_s": PART_C4_ITERS * M / (ms / 1e3), "trace_sha16": trace_sha,
                               "exchange": "device-initiated: red.min.sys / red.release.sys into every GPU's "
                                           "exchange buffer (CUDA IPC), no host step"}
        return part

    if not args.no_partitioned:
        section("partitioned", partitioned)

    # ---- UBQP: k = 3, n = 500 OR-Library-style Q, one search (N = 1 only; context)
    def ubqp_single():
        from ppp_inputs import bqp as bi

        nq, kq, itq = 500, 3, 256  # >= 128 iterations: the CUDA-graph path (64-iteration blocks)
        Qb = bi.random_q(nq, 0.1, 1)
        xq = bi.start_x(nq, 2)
        cq = L.lns_bqp_create(Qb, 0)
        L.lns_bqp_tabu_run(cq, kq, 128, -1, xq, trace=False)
        msq = []
        for _ in range(2):
            flush.fill_(0)
            torch.cuda.synchronize()
            L.lns_bqp_tabu_run(cq, kq, itq, -1, xq, trace=False)
            msq.append(L.lns_bqp_last_kernel_ms(cq))
        L.lns_bqp_destroy(cq)
        bq = min(msq)
        Mq = L.lns_neighborhood_size(nq, kq)
        return {"neighbors_per_s": itq * Mq / (bq / 1e3), "us_per_iteration": 1e3 * bq / itq, "iters": itq,
                "note": "UBQP f = x^T Q x, n = 500, density 0.1, 3-Hamming (2.07e7 neighbours/iteration), one "
                        "search; device time of the replay (eval + apply launches, CUDA graphs of 64 iterations)"}

    if world == 1 and not args.no_ubqp:
        section("ubqp_single_search", ubqp_single)

    # ---- UBQP restarts side by side (lns_bqp_tabu_run_batch): the quality
    #      protocol's shape, 50 starts of n = 200, k = 3 (N = 1 only; context)
    def ubqp_restarts():
        from ppp_inputs import bqp as bi

        nq, kq, Rq, itq = 200, 3, 50, 256
        Qb = bi.random_q(nq, 0.1, 1000)
        X0 = np.stack([bi.start_x(nq, 100 + r) for r in range(Rq)])
        cq = L.lns_bqp_create(Qb, 0)
        L.lns_bqp_tabu_run_batch(cq, kq, X0, 128)
        msq = []
        for _ in range(2):
            flush.fill_(0)
            torch.cuda.synchronize()
            L.lns_bqp_tabu_run_batch(cq, kq, X0, itq)
            msq.append(L.lns_bqp_last_kernel_ms(cq))
        L.lns_bqp_destroy(cq)
        bq = min(msq)
        Mq = L.lns_neighborhood_size(nq, kq)
        return {"neighbors_per_s": Rq * itq * Mq / (bq / 1e3), "tabu_iters_per_s": Rq * itq / (bq / 1e3),
                "restarts": Rq, "iters": itq,
                "note": "UBQP n = 200, density 0.1, 3-Hamming, 50 restarts in one batched call (one grid row per "
                        "restart); device time"}

    if world == 1 and not args.no_ubqp:
        section("ubqp_restarts", ubqp_restarts)

    def cpu_baseline():
        v, ips, it, runs, cores, dt = oracle_sample(args.cpu_budget)
        v1, ips1, it1, runs1, _, dt1 = oracle_sample(args.cpu_budget, nthreads=1, per_run=10)
        return {"value": v, "unit": UNIT, "cores": cores, "kind": "oracle", "cpu_model": cpu_model(),
                "sample": f"{runs} runs x {ITERS} tabu iterations of step 0 of the {CFG} job (same instance, tenure, "
                          f"start vectors), {dt:.1f} s on {cores} OpenMP threads, from-scratch fitness per neighbour",
                "tabu_iters_per_s": ips,
                "single_thread": {"value": v1, "unit": UNIT, "cores": 1, "tabu_iters_per_s": ips1,
                                  "sample": f"first 10 iterations of runs 0..{runs1 - 1} of step 0, {dt1:.1f} s, "
                                            "one thread (the paper's sequential CPU baseline style, PAPER.md:245-248)"}}

    if rank == 0 and world == 1 and not args.no_cpu_baseline:
        section("cpu_baseline", cpu_baseline)
    ctxl.finish()
    L.lns_destroy(ctx)
    if world > 1:
        dist.destroy_process_group()


if __name__ == "__main__":
    main()
