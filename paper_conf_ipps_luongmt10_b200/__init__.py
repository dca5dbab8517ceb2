"""B200-native k-Hamming tabu search for the Permuted Perceptron Problem.

Thin ctypes binding of the C ABI in ``include/lns.h`` (same names, argument marshalling only):
every step of the hot path -- neighbourhood evaluation, best-move selection, the move and the
tabu bookkeeping -- runs in the sm_100a kernels of ``csrc/lns.cu`` inside ``liblns.so``.
There is no CPU fallback: if the library or a CUDA device is missing, calls raise.

Buffers may be numpy arrays (host), torch CPU tensors or torch CUDA tensors; they are passed by
pointer (the library copies host data itself). Paper: Luong, Melab, Talbi, LSPP@IPDPS 2010
(PAPER.md); see DESIGN.md for the readings of the paper this follows.
"""
from __future__ import annotations

import ctypes
import os
from typing import Any, Optional

import numpy as np

from . import _build

LNS_OK = 0
LNS_EINVAL = -1
LNS_ERANGE = -2
LNS_ENOMEM = -3
LNS_ECUDA = -4
LNS_ENCCL = -5
LNS_ENOADMISSIBLE = -6
LNS_EPEER = -7
LNS_STOP_ON_ZERO = 1
LNS_FORCE_STEPPED = 2
LNS_ASPIRATION = 4
LNS_TABU_SOLUTIONS = 16
LNS_PLAIN_LAUNCH = 8
KEY_NONE = (1 << 63) - 1
LNS_IPC_HANDLE_BYTES = 64
LNS_UNIQUE_ID_BYTES = 128

RESULT_FIELDS = ("iters_done", "final_f", "best_f", "best_iter", "first_zero_iter", "solved")


class LnsError(RuntimeError):
    def __init__(self, status: int, where: str, detail: str):
        super().__init__(f"{where}: {detail} (status {status})")
        self.status = status


class lns_result(ctypes.Structure):
    _fields_ = [("iters_done", ctypes.c_int64), ("final_f", ctypes.c_int64), ("best_f", ctypes.c_int64),
                ("best_iter", ctypes.c_int64), ("first_zero_iter", ctypes.c_int64),
                ("solved", ctypes.c_int32), ("reserved", ctypes.c_int32)]

    def as_dict(self) -> dict:
        return {f: int(getattr(self, f)) for f in RESULT_FIELDS}


_lib = None
_vp, _i32, _i64, _u64 = ctypes.c_void_p, ctypes.c_int32, ctypes.c_int64, ctypes.c_uint64
_SIGS = {
    "lns_create": (_i32, [_vp, _i32, _i32, _vp, _i32, ctypes.POINTER(_vp)]),
    "lns_destroy": (None, [_vp]),
    "lns_eval_neighborhood": (_i32, [_vp, _i32, _vp, _vp, _vp, ctypes.POINTER(_i64), ctypes.POINTER(_i64), _vp]),
    "lns_eval_all": (_i32, [_vp, _i32, _vp, _vp, _vp]),
    "lns_tabu_run": (_i32, [_vp, _i32, _i64, _i64, _u64, _vp, _i32, _vp, _vp, _vp, ctypes.POINTER(lns_result), _vp]),
    "lns_tabu_run_batch": (_i32, [_vp, _i32, _i32, _i64, _i64, _u64, _vp, _i32, _vp, _vp, _vp]),
    "lns_unrank": (_i32, [_i32, _i32, _vp, _i64, _vp, _vp]),
    "lns_set_partition": (_i32, [_vp, _i32, _i32]),
    "lns_attach_comm": (_i32, [_vp, _vp, _i32, _i32]),
    "lns_get_unique_id": (_i32, [_vp]),
    "lns_comm_init_rank": (_i32, [_vp, _vp, _i32, _i32]),
    "lns_exchange_buffer": (_i32, [_vp, ctypes.POINTER(_vp)]),
    "lns_exchange_ipc_handle": (_i32, [_vp, _vp]),
    "lns_attach_peers": (_i32, [_vp, _i32, _i32, ctypes.POINTER(_vp), _i64]),
    "lns_attach_peers_ipc": (_i32, [_vp, _i32, _i32, _vp, _i64]),
    "lns_exchange_reset": (_i32, [_vp, _vp]),
    "lns_step_begin": (_i32, [_vp, _i32, _i64, _i64, _u64, _vp, _i32, _vp]),
    "lns_step_eval": (_i32, [_vp, _vp, _vp]),
    "lns_step_apply": (_i32, [_vp, _vp, _vp]),
    "lns_step_end": (_i32, [_vp, _vp, _vp, _vp, ctypes.POINTER(lns_result), _vp]),
    "lns_last_kernel_ms": (ctypes.c_double, [_vp]),
    "lns_config": (_i32, [_vp, _i32]),
    "lns_neighborhood_size": (_i64, [_i32, _i32]),
    "lns_strerror": (ctypes.c_char_p, [_i32]),
    "lns_last_error": (ctypes.c_char_p, []),
    "lns_version": (_i32, []),
    "lns_pool_trim": (None, []),
    "lns_pool_stats": (None, [ctypes.POINTER(_i64), ctypes.POINTER(_i64)]),
    "lns_bqp_create": (_i32, [_vp, _i32, _i32, ctypes.POINTER(_vp)]),
    "lns_bqp_destroy": (None, [_vp]),
    "lns_bqp_eval_all": (_i32, [_vp, _i32, _vp, _vp, _vp]),
    "lns_bqp_tabu_run": (_i32, [_vp, _i32, _i64, _i64, _vp, _vp, _vp, _vp, _vp, _vp]),
    "lns_bqp_tabu_run_batch": (_i32, [_vp, _i32, _i32, _i64, _i64, _vp, _vp, _vp, _vp]),
    "lns_bqp_last_kernel_ms": (ctypes.c_double, [_vp]),
}


def library_path() -> str:
    """liblns.so in the package (LNS_LIB may point at a variant build, e.g. the profiling one)."""
    return os.environ.get("LNS_LIB") or _build.LIB


def load(build_if_missing: bool = True):
    """Load liblns.so (building it with nvcc first if it is missing or stale)."""
    global _lib
    if _lib is None:
        path = library_path()
        if build_if_missing and path == _build.LIB and _build.stale():
            _build.build()
        if not os.path.exists(path):
            raise RuntimeError(f"CUDA extension {path} is missing; run _build.build()")
        lib = ctypes.CDLL(path)
        for name, (res, args) in _SIGS.items():
            fn = getattr(lib, name)
            fn.restype = res
            fn.argtypes = args
        _lib = lib
    return _lib


def _check(status: int, where: str):
    if status != LNS_OK:
        lib = load()
        raise LnsError(status, where, (lib.lns_last_error() or b"").decode() or lib.lns_strerror(status).decode())


# --------------------------------------------------------------------------- marshalling
def _ptr(x, dtype) -> tuple[Optional[int], Any]:
    """(pointer, keep-alive) for numpy arrays / torch tensors; None -> NULL."""
    if x is None:
        return None, None
    if isinstance(x, np.ndarray):
        a = np.ascontiguousarray(x, dtype=dtype)
        return a.ctypes.data, a
    try:
        import torch
    except ImportError:  # pragma: no cover
        torch = None
    if torch is not None and isinstance(x, torch.Tensor):
        tdt = {np.int8: torch.int8, np.uint8: torch.uint8, np.int32: torch.int32, np.int64: torch.int64,
               np.uint32: torch.int32}[dtype]
        t = x.contiguous()
        if t.dtype != tdt:
            t = t.to(tdt)
        return t.data_ptr(), t
    a = np.ascontiguousarray(np.asarray(x), dtype=dtype)
    return a.ctypes.data, a


def _out_ptr(x, dtype):
    """Output buffers must already have the right dtype and be contiguous (written in place)."""
    if x is None:
        return None
    if isinstance(x, np.ndarray):
        assert x.dtype == dtype and x.flags.c_contiguous, "output array must be contiguous " + str(dtype)
        return x.ctypes.data
    import torch

    assert isinstance(x, torch.Tensor) and x.is_contiguous()
    want = {np.int8: torch.int8, np.uint8: torch.uint8, np.int32: torch.int32, np.int64: torch.int64}[dtype]
    assert x.dtype == want, f"output tensor must be {want}"
    return x.data_ptr()


def _stream(stream) -> Optional[int]:
    if stream is None:
        return None
    if isinstance(stream, int):
        return stream
    return int(stream.cuda_stream)  # torch.cuda.Stream


# --------------------------------------------------------------------------- C ABI, same names
def lns_version() -> int:
    return int(load().lns_version())


def lns_pool_trim() -> None:
    """Release the library's cached device blocks (include/lns.h, device-memory cache)."""
    load().lns_pool_trim()


def lns_pool_stats() -> tuple[int, int]:
    """(cached bytes, live bytes) of the library's device-memory cache."""
    c, l_ = _i64(0), _i64(0)
    load().lns_pool_stats(ctypes.byref(c), ctypes.byref(l_))
    return int(c.value), int(l_.value)


def lns_strerror(status: int) -> str:
    return load().lns_strerror(status).decode()


def lns_neighborhood_size(n: int, k: int) -> int:
    return int(load().lns_neighborhood_size(n, k))


def lns_create(A, S, device: int = 0) -> int:
    """Upload an instance (A: m x n of +-1, S: m ints in [0, n]); returns the context handle."""
    shape = tuple(A.shape)
    m, n = int(shape[0]), int(shape[1])
    pa, ka = _ptr(A, np.int8)
    ps, ks = _ptr(S, np.int32)
    out = _vp()
    _check(load().lns_create(pa, m, n, ps, device, ctypes.byref(out)), "lns_create")
    return out.value


def lns_destroy(ctx: int) -> None:
    load().lns_destroy(ctx)


def lns_config(ctx: int, blocks: int = 0) -> None:
    _check(load().lns_config(ctx, blocks), "lns_config")


def lns_last_kernel_ms(ctx: int) -> float:
    return float(load().lns_last_kernel_ms(ctx))


def lns_set_partition(ctx: int, part: int, nparts: int) -> None:
    _check(load().lns_set_partition(ctx, part, nparts), "lns_set_partition")


def lns_attach_comm(ctx: int, comm_ptr: Optional[int], rank: int, world: int) -> None:
    _check(load().lns_attach_comm(ctx, comm_ptr, rank, world), "lns_attach_comm")


def lns_get_unique_id() -> bytes:
    """A fresh ncclUniqueId (LNS_UNIQUE_ID_BYTES) for lns_comm_init_rank (call on one rank)."""
    buf = ctypes.create_string_buffer(LNS_UNIQUE_ID_BYTES)
    _check(load().lns_get_unique_id(buf), "lns_get_unique_id")
    return buf.raw


def lns_comm_init_rank(ctx: int, uid: bytes, rank: int, world: int) -> None:
    """Create (collectively over `world` processes) an NCCL communicator owned by ctx and attach it."""
    if len(uid) != LNS_UNIQUE_ID_BYTES:
        raise ValueError("uid must be LNS_UNIQUE_ID_BYTES long")
    buf = ctypes.create_string_buffer(bytes(uid), LNS_UNIQUE_ID_BYTES)
    _check(load().lns_comm_init_rank(ctx, buf, rank, world), "lns_comm_init_rank")


def lns_exchange_buffer(ctx: int) -> int:
    """Device pointer of this context's 512-byte exchange buffer (device-initiated exchange)."""
    p = _vp()
    _check(load().lns_exchange_buffer(ctx, ctypes.byref(p)), "lns_exchange_buffer")
    return int(p.value)


def lns_exchange_ipc_handle(ctx: int) -> bytes:
    """cudaIpcMemHandle_t (LNS_IPC_HANDLE_BYTES) of the exchange buffer, for other processes."""
    buf = ctypes.create_string_buffer(LNS_IPC_HANDLE_BYTES)
    _check(load().lns_exchange_ipc_handle(ctx, buf), "lns_exchange_ipc_handle")
    return buf.raw


def lns_attach_peers(ctx: int, part: int, nparts: int, bufs, timeout_ms: int = 10000) -> None:
    """Partition `part` of `nparts` with the partitions' exchange buffers (device pointers usable
    from this context's device); nparts = 1 / bufs = None detaches."""
    arr = None
    if bufs is not None:
        arr = (_vp * len(bufs))(*[int(b) for b in bufs])
    _check(load().lns_attach_peers(ctx, part, nparts, arr, timeout_ms), "lns_attach_peers")


def lns_attach_peers_ipc(ctx: int, part: int, nparts: int, handles: bytes, timeout_ms: int = 10000) -> None:
    """As lns_attach_peers from the concatenated IPC handles of all partitions (one process per GPU)."""
    if len(handles) != nparts * LNS_IPC_HANDLE_BYTES:
        raise ValueError("handles must hold nparts x LNS_IPC_HANDLE_BYTES bytes")
    buf = ctypes.create_string_buffer(handles, len(handles))
    _check(load().lns_attach_peers_ipc(ctx, part, nparts, buf, timeout_ms), "lns_attach_peers_ipc")


def lns_exchange_reset(ctx: int, stream=None) -> None:
    """Clear this context's exchange buffer (before every peer run, then a host barrier)."""
    _check(load().lns_exchange_reset(ctx, _stream(stream)), "lns_exchange_reset")


def lns_eval_neighborhood(ctx: int, k: int, V, Y, tabu_bits=None, stream=None) -> tuple[int, int]:
    """(best fitness, best rank) over admissible neighbours; raises LnsError(ENOADMISSIBLE)."""
    pv, kv = _ptr(V, np.int8)
    py, ky = _ptr(Y, np.int32)
    pt, kt = _ptr(tabu_bits, np.uint32)
    bf, br = _i64(), _i64()
    _check(load().lns_eval_neighborhood(ctx, k, pv, py, pt, ctypes.byref(bf), ctypes.byref(br), _stream(stream)),
           "lns_eval_neighborhood")
    return int(bf.value), int(br.value)


def lns_eval_all(ctx: int, k: int, V, out=None, stream=None):
    """Fitness of every neighbour by rank (int32); `out` may be a device tensor."""
    if out is None:
        n = len(V)
        out = np.empty(lns_neighborhood_size(n, k), dtype=np.int32)
    pv, kv = _ptr(V, np.int8)
    _check(load().lns_eval_all(ctx, k, pv, _out_ptr(out, np.int32), _stream(stream)), "lns_eval_all")
    return out


def lns_tabu_run(ctx: int, k: int, iters: int, tenure: int = -1, seed: int = 0, V0=None,
                 flags: int = LNS_STOP_ON_ZERO, V_out=None, trace_rank=None, trace_fit=None, stream=None) -> dict:
    pv, kv = _ptr(V0, np.int8)
    res = lns_result()
    _check(load().lns_tabu_run(ctx, k, iters, tenure, seed & ((1 << 64) - 1), pv, flags, _out_ptr(V_out, np.int8),
                               _out_ptr(trace_rank, np.int64), _out_ptr(trace_fit, np.int64), ctypes.byref(res),
                               _stream(stream)), "lns_tabu_run")
    return res.as_dict()


def lns_tabu_run_batch(ctx: int, k: int, R: int, iters: int, tenure: int = -1, seed: int = 0, V0=None,
                       flags: int = LNS_STOP_ON_ZERO, V_out=None, stream=None) -> list[dict]:
    pv, kv = _ptr(V0, np.int8)
    res = (lns_result * max(R, 1))()
    _check(load().lns_tabu_run_batch(ctx, k, R, iters, tenure, seed & ((1 << 64) - 1), pv, flags,
                                     _out_ptr(V_out, np.int8), res, _stream(stream)), "lns_tabu_run_batch")
    return [res[i].as_dict() for i in range(R)]


def lns_unrank(n: int, k: int, ranks, out=None, stream=None):
    pr, kr = _ptr(ranks, np.int64)
    cnt = int(len(ranks))
    if out is None:
        out = np.empty((cnt, max(3, k)), dtype=np.int32)  # k >= 4: count x k
    _check(load().lns_unrank(n, k, pr, cnt, _out_ptr(out, np.int32), _stream(stream)), "lns_unrank")
    return out


def lns_step_begin(ctx: int, k: int, max_iters: int, tenure: int = -1, seed: int = 0, V0=None,
                   flags: int = LNS_STOP_ON_ZERO, stream=None) -> None:
    pv, kv = _ptr(V0, np.int8)
    _check(load().lns_step_begin(ctx, k, max_iters, tenure, seed & ((1 << 64) - 1), pv, flags, _stream(stream)),
           "lns_step_begin")


def lns_step_eval(ctx: int, key_dev, stream=None) -> None:
    """key_dev: a CUDA int64 tensor (>= 1 element) that receives the partial best key."""
    _check(load().lns_step_eval(ctx, _out_ptr(key_dev, np.int64), _stream(stream)), "lns_step_eval")


def lns_step_apply(ctx: int, key_dev, stream=None) -> None:
    _check(load().lns_step_apply(ctx, _out_ptr(key_dev, np.int64), _stream(stream)), "lns_step_apply")


def lns_step_end(ctx: int, V_out=None, trace_rank=None, trace_fit=None, stream=None) -> dict:
    res = lns_result()
    _check(load().lns_step_end(ctx, _out_ptr(V_out, np.int8), _out_ptr(trace_rank, np.int64),
                               _out_ptr(trace_fit, np.int64), ctypes.byref(res), _stream(stream)), "lns_step_end")
    return res.as_dict()


class Instance:
    """RAII wrapper of an lns context (owning the handle)."""

    def __init__(self, A, S, device: int = 0):
        self.m, self.n = int(A.shape[0]), int(A.shape[1])
        self.ctx = lns_create(A, S, device)

    def close(self):
        if getattr(self, "ctx", None):
            lns_destroy(self.ctx)
            self.ctx = None

    def __del__(self):
        try:
            self.close()
        except Exception:
            pass

    def __enter__(self):
        return self

    def __exit__(self, *exc):
        self.close()

    def tabu_run(self, k, iters, tenure=-1, seed=0, V0=None, stop_on_zero=True, trace=True, stream=None, flags=0):
        tr = np.full(max(iters, 1), -1, np.int64) if trace else None
        tf = np.full(max(iters, 1), -1, np.int64) if trace else None
        Vo = np.empty(self.n, np.int8)
        fl = (LNS_STOP_ON_ZERO if stop_on_zero else 0) | flags
        res = lns_tabu_run(self.ctx, k, iters, tenure, seed, V0, fl, Vo, tr, tf, stream)
        it = res["iters_done"]
        return (tr[:it] if trace else None), (tf[:it] if trace else None), Vo, res


# --------------------------------------------------------------------------- UBQP
BQP_RESULT_FIELDS = ("iters_done", "final_f", "best_f", "best_iter")


def lns_bqp_create(Q, device: int = 0) -> int:
    """Upload a symmetric int32 n x n matrix Q (f(x) = x^T Q x, x in {0,1}^n); returns the handle."""
    n = int(tuple(Q.shape)[0])
    pq, kq = _ptr(Q, np.int32)
    out = _vp()
    _check(load().lns_bqp_create(pq, n, device, ctypes.byref(out)), "lns_bqp_create")
    return out.value


def lns_bqp_destroy(ctx: int) -> None:
    load().lns_bqp_destroy(ctx)


def lns_bqp_eval_all(ctx: int, k: int, x, out=None, stream=None):
    """f(x xor F_r) for every rank r (int32); `out` may be a device tensor."""
    if out is None:
        out = np.empty(lns_neighborhood_size(len(x), k), dtype=np.int32)
    px, kx = _ptr(x, np.uint8)
    _check(load().lns_bqp_eval_all(ctx, k, px, _out_ptr(out, np.int32), _stream(stream)), "lns_bqp_eval_all")
    return out


def lns_bqp_tabu_run(ctx: int, k: int, iters: int, tenure: int = -1, x0=None, x_out=None,
                     trace: bool = True, stream=None):
    """(trace_rank, trace_fit, x_out, result dict) of `iters` tabu iterations from x0 (uint8 0/1)."""
    n = len(x0)
    px, kx = _ptr(x0, np.uint8)
    if x_out is None:
        x_out = np.empty(n, dtype=np.uint8)
    tr = np.empty(max(iters, 1), dtype=np.int64) if trace else None
    tf = np.empty(max(iters, 1), dtype=np.int64) if trace else None
    res = np.zeros(4, dtype=np.int64)
    _check(load().lns_bqp_tabu_run(ctx, k, iters, tenure, px, _out_ptr(x_out, np.uint8),
                                   None if tr is None else tr.ctypes.data,
                                   None if tf is None else tf.ctypes.data, res.ctypes.data, _stream(stream)),
           "lns_bqp_tabu_run")
    d = dict(zip(BQP_RESULT_FIELDS, (int(v) for v in res)))
    it = d["iters_done"]
    return (None if tr is None else tr[:it].copy()), (None if tf is None else tf[:it].copy()), x_out, d


def lns_bqp_tabu_run_batch(ctx: int, k: int, x0s, iters: int, tenure: int = -1, x_outs=None, stream=None):
    """R = len(x0s) independent tabu searches run side by side (x0s: R x n uint8 0/1); returns one
    result dict per restart (the fields of lns_bqp_tabu_run); x_outs (R x n) receives the final x."""
    R = int(tuple(x0s.shape)[0])
    px, kx = _ptr(x0s, np.uint8)
    res = np.zeros((max(R, 1), 4), dtype=np.int64)
    _check(load().lns_bqp_tabu_run_batch(ctx, k, R, iters, tenure, px, _out_ptr(x_outs, np.uint8),
                                         res.ctypes.data, _stream(stream)), "lns_bqp_tabu_run_batch")
    return [dict(zip(BQP_RESULT_FIELDS, (int(v) for v in row))) for row in res[:R]]


def lns_bqp_last_kernel_ms(ctx: int) -> float:
    return float(load().lns_bqp_last_kernel_ms(ctx))
