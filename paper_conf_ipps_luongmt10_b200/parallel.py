"""Multi-GPU drivers of the k-Hamming tabu search (one process per GPU, torch.distributed).

Two ways to use several GPUs, both from SURVEY.md §8(e) / DESIGN.md §8:

* **Partitioned search** ("partitioning the neighborhood set, where each
  partition is executed on a single GPU"). GPU g evaluates ranks [B(g), B(g+1)) of the
  neighbourhood (``slice_bounds``); per iteration the partial best keys ((fitness << 32) | rank)
  are combined by ONE all-reduce MIN of a single int64 and every GPU applies the same move. The
  trajectory is identical for any number of GPUs (a MIN over exact keys is associative). The
  production path is ``lns_tabu_run`` with ``lns_attach_comm`` (the loop and ncclAllReduce run in
  C); ``partitioned_tabu_run`` below is the same protocol driven from Python over any
  ``Stepper`` and any torch.distributed backend (it is what the gloo tests exercise).
* **Independent restarts**: restart r runs on rank r mod world (``restart_shard``); no data-path
  collective, only a final gather of the per-restart results (``sharded_restarts``).
* **Device-initiated exchange** (``peer_tabu_run``): the partitioned search
  with the per-iteration MIN done by the persistent kernels themselves -- every CTA MINs its key
  into every GPU's exchange buffer over NVLink peer memory and waits on its own arrival counter --
  so there is no host collective and no per-iteration launch. Buffers are shared once per run as
  CUDA IPC handles (``gather_exchange_handles``).

Nothing here computes on the CPU: the GPU ``LnsStepper`` drives the kernels of liblns.so.
"""
from __future__ import annotations

from typing import Callable, Optional, Protocol

import torch
import torch.distributed as dist

KEY_NONE = (1 << 63) - 1


def slice_bounds(M: int, part: int, nparts: int) -> tuple[int, int]:
    """Rank slice of partition `part` (same formula as the C library, include/lns.h):
    B(g) = 32 * floor(M g / (32 nparts)), B(nparts) = M."""
    if not (0 <= part < nparts):
        raise ValueError("bad partition")

    def B(g):
        return M if g >= nparts else 32 * ((M * g // nparts) // 32)

    return B(part), B(part + 1)


def pack_key(f: int, r: int) -> int:
    """The 63-bit selection key: least fitness first, lowest rank on ties (R5)."""
    return (int(f) << 32) | int(r)


def unpack_key(key: int) -> tuple[int, int]:
    return int(key) >> 32, int(key) & 0xFFFFFFFF


class Stepper(Protocol):
    """One partition of a stepped search (see include/lns.h, lns_step_*)."""

    def key_buffer(self) -> torch.Tensor: ...

    def eval(self, key: torch.Tensor) -> None: ...

    def apply(self, key: torch.Tensor) -> None: ...

    def done(self) -> bool: ...

    def end(self): ...


def partitioned_tabu_run(stepper: Stepper, iters: int, group=None, check_every: int = 64):
    """Run `iters` iterations of the partitioned protocol: local evaluation of this rank's slice,
    all-reduce MIN of the int64 key, identical move everywhere. Returns ``stepper.end()``."""
    key = stepper.key_buffer()
    for t in range(iters):
        stepper.eval(key)
        dist.all_reduce(key, op=dist.ReduceOp.MIN, group=group)
        stepper.apply(key)
        if check_every and (t + 1) % check_every == 0 and stepper.done():
            break
    return stepper.end()


class LnsStepper:
    """GPU stepper over liblns.so for partition (rank, world) of the rank space."""

    def __init__(self, ctx: int, n: int, k: int, iters: int, tenure: int = -1, seed: int = 0, V0=None,
                 stop_on_zero: bool = True, rank: int = 0, world: int = 1, device: Optional[torch.device] = None):
        from . import LNS_STOP_ON_ZERO, lns_set_partition, lns_step_begin

        self.ctx, self.iters, self.n = ctx, iters, n
        self.device = device or torch.device("cuda", torch.cuda.current_device())
        lns_set_partition(ctx, rank, world)
        lns_step_begin(ctx, k, iters, tenure, seed, V0, LNS_STOP_ON_ZERO if stop_on_zero else 0)
        self._key = torch.full((1,), KEY_NONE, dtype=torch.int64, device=self.device)
        self._n = None

    def key_buffer(self) -> torch.Tensor:
        return self._key

    def eval(self, key):
        from . import lns_step_eval

        lns_step_eval(self.ctx, key)

    def apply(self, key):
        from . import lns_step_apply

        lns_step_apply(self.ctx, key)

    def done(self) -> bool:
        return False  # the device turns iterations after f = 0 into no-ops

    def end(self):
        import numpy as np

        from . import lns_step_end

        tr = np.full(max(self.iters, 1), -1, np.int64)
        tf = np.full(max(self.iters, 1), -1, np.int64)
        Vo = np.empty(self.n, np.int8)
        res = lns_step_end(self.ctx, Vo, tr, tf)
        it = res["iters_done"]
        return tr[:it], tf[:it], Vo, res


def nccl_comm_ptr(group=None, device: Optional[torch.device] = None) -> int:
    """The ncclComm_t of a torch NCCL process group (for lns_attach_comm): torch's own libnccl
    created it, and lns_attach_comm looks ncclAllReduce up in that same loaded copy."""
    device = device or torch.device("cuda", torch.cuda.current_device())
    pg = group or dist.group.WORLD
    backend = pg._get_backend(device)
    # make sure the communicator exists (torch creates it lazily unless device_id was given)
    t = torch.zeros(1, device=device)
    dist.all_reduce(t, group=pg)
    torch.cuda.synchronize(device)
    ptr = int(backend._comm_ptr())
    if not ptr:
        raise RuntimeError("no NCCL communicator behind this process group")
    return ptr


def restart_shard(R: int, rank: int, world: int) -> list[int]:
    """Restarts owned by `rank`: r = rank, rank + world, ... (restart r on GPU r mod world)."""
    return list(range(rank, R, world))


def sharded_restarts(run_one: Callable[[int], dict], R: int, group=None) -> list[dict]:
    """Run the restarts of this rank with run_one(r) and gather every rank's results in restart
    order (only a final all_gather_object; no per-iteration communication)."""
    rank = dist.get_rank(group) if dist.is_initialized() else 0
    world = dist.get_world_size(group) if dist.is_initialized() else 1
    mine = {r: run_one(r) for r in restart_shard(R, rank, world)}
    if world == 1:
        return [mine[r] for r in range(R)]
    parts: list = [None] * world
    dist.all_gather_object(parts, mine, group=group)
    merged = {}
    for p in parts:
        merged.update(p)
    return [merged[r] for r in range(R)]


# ------------------------------------------------------------------ device-initiated exchange (f3)
def gather_exchange_handles(handle: bytes, group=None) -> bytes:
    """Every rank's exchange-buffer IPC handle, concatenated in rank order (what
    lns_attach_peers_ipc takes). Pure host logic: works over gloo or NCCL process groups."""
    world = dist.get_world_size(group) if dist.is_initialized() else 1
    if world == 1:
        return bytes(handle)
    got = [None] * world
    dist.all_gather_object(got, bytes(handle), group=group)
    if any(len(h) != len(handle) for h in got):
        raise ValueError("exchange handles differ in size across ranks")
    return b"".join(got)


def peer_tabu_run(ctx: int, k: int, iters: int, tenure: int = -1, seed: int = 0, V0=None, flags: int = 0,
                  group=None, timeout_ms: int = 10000, V_out=None, trace_rank=None, trace_fit=None, stream=None):
    """One search over all ranks of `group`, one process per GPU, with the per-iteration argmin
    exchanged by the persistent kernels themselves through NVLink peer memory (lns_attach_peers_ipc;
    SURVEY.md §8(f) f3) instead of a host all-reduce. Rank r evaluates slice r of the rank space;
    the trajectory equals the single-GPU one. Returns this rank's lns_tabu_run result dict (outputs
    as in lns_tabu_run)."""
    from . import (lns_attach_peers, lns_attach_peers_ipc, lns_exchange_ipc_handle, lns_exchange_reset,
                   lns_tabu_run)
    rank = dist.get_rank(group) if dist.is_initialized() else 0
    world = dist.get_world_size(group) if dist.is_initialized() else 1
    if world > 1:
        handles = gather_exchange_handles(lns_exchange_ipc_handle(ctx), group)
        lns_attach_peers_ipc(ctx, rank, world, handles, timeout_ms)
        lns_exchange_reset(ctx, stream)
        dist.barrier(group)  # every partition's buffer is clear before any kernel starts
    try:
        return lns_tabu_run(ctx, k, iters, tenure, seed, V0, flags, V_out, trace_rank, trace_fit, stream)
    finally:
        if world > 1:
            lns_attach_peers(ctx, 0, 1, None)
