"""The N > 1 host logic on CPU: world-size-2 (and 3) gloo process groups.

The partitioned protocol (slice evaluation, all-reduce MIN of the 63-bit key, identical move on
every rank) and restart sharding are driven exactly as on GPUs, with the oracle standing in for
the per-slice evaluation. The resulting trajectory must equal the single-process oracle run.
"""
import os
import socket
from math import comb

import numpy as np
import pytest
import torch
import torch.distributed as dist
import torch.multiprocessing as mp

import ppp_inputs as pi
from paper_conf_ipps_luongmt10_b200 import parallel as par


def _free_port():
    with socket.socket() as s:
        s.bind(("127.0.0.1", 0))
        return s.getsockname()[1]


class OracleSliceStepper:
    """CPU stand-in for one GPU partition: evaluates its slice with the oracle."""

    def __init__(self, A, S, k, V0, iters, tenure, rank, world, stop_on_zero=True):
        import oracle

        self.o = oracle
        self.A, self.S, self.k = A, S, k
        self.n = A.shape[1]
        self.M = comb(self.n, k)
        self.lo, self.hi = par.slice_bounds(self.M, rank, world)
        self.L = tenure
        self.V = np.array(V0, np.int8)
        self.f = oracle.fitness(A, S, self.V)
        self.until = np.zeros(self.M, np.int64)  # only this slice is ever written
        self.t = 0
        self.iters, self.stop = iters, stop_on_zero
        self.trace_r, self.trace_f = [], []
        self.finished = stop_on_zero and self.f == 0

    def key_buffer(self):
        return torch.full((1,), par.KEY_NONE, dtype=torch.int64)

    def eval(self, key):
        if self.finished:
            key[0] = par.KEY_NONE
            return
        t = self.t + 1
        fa = self.o.eval_all(self.A, self.S, self.V, self.k, nthreads=1)
        best = par.KEY_NONE
        for r in range(self.lo, self.hi):
            if self.until[r] < t:
                best = min(best, par.pack_key(fa[r], r))
        key[0] = best

    def apply(self, key):
        if self.finished:
            return
        f, r = par.unpack_key(int(key[0]))
        self.t += 1
        (fs,) = self.o.flipsets(self.n, self.k, [r])
        for i in fs:
            if i >= 0:
                self.V[i] = -self.V[i]
        if self.lo <= r < self.hi:
            self.until[r] = self.t + self.L
        self.f = f
        self.trace_r.append(r)
        self.trace_f.append(f)
        if (self.stop and f == 0) or self.t >= self.iters:
            self.finished = True

    def done(self):
        return self.finished

    def end(self):
        return np.array(self.trace_r), np.array(self.trace_f), self.V.copy(), self.f


def _worker(rank, world, port, cfg, out):
    os.environ.update(MASTER_ADDR="127.0.0.1", MASTER_PORT=str(port))
    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        if cfg["kind"] == "partition":
            inst = pi.planted_instance(cfg["m"], cfg["n"], cfg["seed"])
            V0 = pi.start_vector(cfg["n"], cfg["vseed"])
            st = OracleSliceStepper(inst.A, inst.S, cfg["k"], V0, cfg["iters"], cfg["tenure"], rank, world,
                                    cfg["stop"])
            tr, tf, V, f = par.partitioned_tabu_run(st, cfg["iters"], check_every=1)
            out[rank] = (tr.tolist(), tf.tolist(), V.tolist(), f)
        elif cfg["kind"] == "restarts":
            import oracle

            inst = pi.planted_instance(cfg["m"], cfg["n"], cfg["seed"])

            def run_one(r):
                V0 = pi.start_vector(cfg["n"], pi.restart_seed(cfg["vseed"], r))
                _, _, _, res = oracle.tabu_run(inst.A, inst.S, cfg["k"], V0, cfg["iters"], cfg["tenure"],
                                               nthreads=1)
                res["rank"] = rank
                return res

            out[rank] = par.sharded_restarts(run_one, cfg["R"])
        if cfg["kind"] == "handles":
            # each rank's (fake) 64-byte IPC handle; every rank must get all, in rank order
            mine = bytes([rank + 1]) * 64
            out[rank] = par.gather_exchange_handles(mine)
    finally:
        dist.destroy_process_group()


def _spawn(world, cfg):
    mgr = mp.Manager()
    out = mgr.dict()
    mp.spawn(_worker, args=(world, _free_port(), cfg, out), nprocs=world, join=True)
    return dict(out)


def test_slice_bounds_partition_the_rank_space():
    for M in (1, 21, 33, 2628, 85320, 260130, 178433024):
        for G in (1, 2, 3, 4, 7, 8):
            b = [par.slice_bounds(M, g, G) for g in range(G)]
            assert b[0][0] == 0 and b[-1][1] == M
            for (lo, hi), (lo2, _) in zip(b, b[1:]):
                assert hi == lo2 and lo % 32 == 0
            assert all(lo <= hi for lo, hi in b)


def test_key_order_is_fitness_then_rank():
    keys = [par.pack_key(f, r) for f, r in [(5, 9), (5, 3), (4, 100), (6, 0)]]
    assert min(keys) == par.pack_key(4, 100)
    assert sorted(keys)[1] == par.pack_key(5, 3)
    assert par.unpack_key(par.pack_key(123456, 4000000000)) == (123456, 4000000000)


@pytest.mark.parametrize("world,k,tenure", [(2, 1, 3), (2, 3, 200), (3, 2, 50)])
def test_partitioned_search_gloo_matches_single_process(orc, world, k, tenure):
    cfg = dict(kind="partition", m=23, n=19, k=k, seed=77 + k, vseed=5, iters=25, tenure=tenure, stop=False)
    out = _spawn(world, cfg)
    inst = pi.planted_instance(23, 19, 77 + k)
    tr, tf, Vo, res = orc.tabu_run(inst.A, inst.S, k, pi.start_vector(19, 5), 25, tenure, stop_on_zero=False)
    for rank in range(world):
        rtr, rtf, rV, rf = out[rank]
        assert rtr == tr.tolist() and rtf == tf.tolist()
        assert rV == Vo.tolist() and rf == res["final_f"]


def test_partitioned_search_gloo_stop_on_zero(orc):
    cfg = dict(kind="partition", m=21, n=21, k=1, seed=1001, vseed=2, iters=200, tenure=3, stop=True)
    out = _spawn(2, cfg)
    inst = pi.config_instance("C1")
    tr, tf, Vo, res = orc.tabu_run(inst.A, inst.S, 1, pi.start_vector(21, 2), 200, 3, stop_on_zero=True)
    assert res["solved"]
    for rank in range(2):
        assert out[rank][0] == tr.tolist() and out[rank][3] == 0


def test_sharded_restarts_gloo(orc):
    cfg = dict(kind="restarts", m=21, n=21, k=1, seed=1001, vseed=9, iters=300, tenure=3, R=5)
    out = _spawn(2, cfg)
    inst = pi.config_instance("C1")
    for rank in range(2):
        got = out[rank]
        assert [g["rank"] for g in got] == [r % 2 for r in range(5)]
        for r, g in enumerate(got):
            V0 = pi.start_vector(21, pi.restart_seed(9, r))
            _, _, _, res = orc.tabu_run(inst.A, inst.S, 1, V0, 300, 3)
            assert {key: g[key] for key in res} == res


@pytest.mark.parametrize("world", [2, 3])
def test_gather_exchange_handles_gloo(world):
    """Host side of the device-initiated exchange (f3): the partitions' exchange-buffer IPC handles
    are gathered in rank order, which is what lns_attach_peers_ipc indexes by partition."""
    out = _spawn(world, dict(kind="handles"))
    want = b"".join(bytes([r + 1]) * 64 for r in range(world))
    for rank in range(world):
        assert out[rank] == want
