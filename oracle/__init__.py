"""CPU oracle for the PPP k-Hamming tabu search -- TEST INFRASTRUCTURE ONLY.

Only ``tests/``, ``__graft_entry__.smoke()`` and ``bench.py``'s ``cpu_baseline`` /
``--impl reference`` legs may import this package. It shares no code with the CUDA path and
never imports ``paper_conf_ipps_luongmt10_b200``. The arithmetic lives in ``oracle.c`` (plain
C, from-scratch fitness for every neighbour, nested-loop enumeration, literal tabu "until"
array); this file only compiles it with gcc and marshals arguments through ctypes.

Parity status of each function: see the header of oracle.c and DESIGN.md §4.
"""
from __future__ import annotations

import ctypes
import os
import subprocess
from math import comb

import numpy as np

_HERE = os.path.dirname(os.path.abspath(__file__))
_SRC = os.path.join(_HERE, "oracle.c")
_LIB = os.path.join(_HERE, "liboracle.so")
_lib = None

_i8p = ctypes.POINTER(ctypes.c_int8)
_i32p = ctypes.POINTER(ctypes.c_int32)
_i64p = ctypes.POINTER(ctypes.c_int64)
_u8p = ctypes.POINTER(ctypes.c_uint8)


def build(force: bool = False) -> str:
    """Compile oracle.c into liboracle.so (gcc -O2 -fopenmp)."""
    if force or not os.path.exists(_LIB) or os.path.getmtime(_LIB) < os.path.getmtime(_SRC):
        tmp = _LIB + f".tmp{os.getpid()}"
        subprocess.check_call(
            ["gcc", "-O2", "-march=x86-64-v2", "-fopenmp", "-shared", "-fPIC", "-std=c11",
             "-Wall", "-o", tmp, _SRC])
        os.replace(tmp, _LIB)
    return _LIB


def _load():
    global _lib
    if _lib is None:
        build()
        lib = ctypes.CDLL(_LIB)
        i32, i64, u64 = ctypes.c_int32, ctypes.c_int64, ctypes.c_uint64
        sig = {
            "oracle_splitmix64_next": (u64, [ctypes.POINTER(u64)]),
            "oracle_start_vector": (None, [i32, u64, _i8p]),
            "oracle_fitness": (i64, [_i8p, i32, i32, _i32p, _i8p]),
            "oracle_fitness_packed": (i64, [_i8p, i32, i32, _i32p, _i8p]),
            "oracle_neighborhood_size": (i64, [i32, i32]),
            "oracle_flipsets": (i32, [i32, i32, _i64p, i64, _i32p]),
            "oracle_eval_all": (i32, [_i8p, i32, i32, _i32p, _i8p, i32, _i64p, i32]),
            "oracle_eval_ranks": (i32, [_i8p, i32, i32, _i32p, _i8p, i32, _i64p, i64, _i64p, i32]),
            "oracle_eval_best": (i32, [_i8p, i32, i32, _i32p, _i8p, i32, _u8p, _i64p, _i64p, i32]),
            "oracle_tabu_run": (i32, [_i8p, i32, i32, _i32p, i32, _i8p, i64, i64, i32, _i64p, _i64p,
                                      _i8p, _i64p, i32, i32]),
            "oracle_max_threads": (i32, []),
        }
        for name, (res, args) in sig.items():
            fn = getattr(lib, name)
            fn.restype = res
            fn.argtypes = args
        _lib = lib
    return _lib


def _p(a: np.ndarray, t):
    return a.ctypes.data_as(t)


def _prep(A, S):
    A = np.ascontiguousarray(A, dtype=np.int8)
    S = np.ascontiguousarray(S, dtype=np.int32)
    m, n = A.shape
    assert S.shape == (m,)
    return A, S, int(m), int(n)


def max_threads() -> int:
    return int(_load().oracle_max_threads())


def splitmix64(state: int, count: int) -> list[int]:
    s = ctypes.c_uint64(state)
    return [int(_load().oracle_splitmix64_next(ctypes.byref(s))) for _ in range(count)]


def start_vector(n: int, seed: int) -> np.ndarray:
    V = np.empty(n, dtype=np.int8)
    _load().oracle_start_vector(n, seed, _p(V, _i8p))
    return V


def fitness(A, S, V, packed: bool = False) -> int:
    """f(V) of PAPER.md:231-237, from scratch (scalar int8 path, or the popcount identity)."""
    A, S, m, n = _prep(A, S)
    V = np.ascontiguousarray(V, dtype=np.int8)
    fn = _load().oracle_fitness_packed if packed else _load().oracle_fitness
    return int(fn(_p(A, _i8p), m, n, _p(S, _i32p), _p(V, _i8p)))


def neighborhood_size(n: int, k: int) -> int:
    return int(_load().oracle_neighborhood_size(n, k))


def flipsets(n: int, k: int, ranks) -> np.ndarray:
    """Flip sets (rows of max(3, k), -1 padded) of ascending `ranks`, by walking the nested loops
    (k >= 4: the odometer generalisation of the same loops)."""
    ranks = np.ascontiguousarray(ranks, dtype=np.int64)
    assert np.all(np.diff(ranks) >= 0)
    out = np.empty((len(ranks), max(3, k)), dtype=np.int32)
    rc = _load().oracle_flipsets(n, k, _p(ranks, _i64p), len(ranks), _p(out, _i32p))
    if rc != 0:
        raise ValueError("rank out of range")
    return out


def eval_all(A, S, V, k: int, nthreads: int = 0) -> np.ndarray:
    """Fitness of every neighbour, index = lexicographic rank (Figs. 7/9/10 new_fitness[])."""
    A, S, m, n = _prep(A, S)
    V = np.ascontiguousarray(V, dtype=np.int8)
    out = np.empty(comb(n, k), dtype=np.int64)
    rc = _load().oracle_eval_all(_p(A, _i8p), m, n, _p(S, _i32p), _p(V, _i8p), k, _p(out, _i64p), nthreads)
    if rc != 0:
        raise ValueError("bad k/n")
    return out


def eval_ranks(A, S, V, k: int, ranks, nthreads: int = 0) -> np.ndarray:
    """Fitness of the neighbours with the given (ascending) ranks."""
    A, S, m, n = _prep(A, S)
    V = np.ascontiguousarray(V, dtype=np.int8)
    ranks = np.ascontiguousarray(ranks, dtype=np.int64)
    assert np.all(np.diff(ranks) >= 0)
    out = np.empty(len(ranks), dtype=np.int64)
    rc = _load().oracle_eval_ranks(_p(A, _i8p), m, n, _p(S, _i32p), _p(V, _i8p), k, _p(ranks, _i64p),
                                   len(ranks), _p(out, _i64p), nthreads)
    if rc != 0:
        raise ValueError("bad k/n")
    return out


def eval_best(A, S, V, k: int, tabu=None, nthreads: int = 0) -> tuple[int, int]:
    """(best fitness, best rank) over admissible neighbours; tabu: bool array of length C(n,k)."""
    A, S, m, n = _prep(A, S)
    V = np.ascontiguousarray(V, dtype=np.int8)
    tp = None
    if tabu is not None:
        tabu = np.ascontiguousarray(tabu, dtype=np.uint8)
        assert tabu.shape == (comb(n, k),)
        tp = _p(tabu, _u8p)
    bf, br = ctypes.c_int64(), ctypes.c_int64()
    _load().oracle_eval_best(_p(A, _i8p), m, n, _p(S, _i32p), _p(V, _i8p), k, tp,
                             ctypes.byref(bf), ctypes.byref(br), nthreads)
    return int(bf.value), int(br.value)


RESULT_FIELDS = ("iters_done", "final_f", "best_f", "best_iter", "first_zero_iter", "solved")


def tabu_run(A, S, k: int, V0, iters: int, tenure: int, stop_on_zero: bool = True, nthreads: int = 0,
             aspiration: bool = False, tabu_solutions: bool = False):
    """Tabu search of PAPER.md:241-258. Returns (trace_rank, trace_fit, V_out, result dict).
    aspiration: a tabu move is admissible when it beats the best fitness so far (variant R4').
    tabu_solutions: the tabu list holds the `tenure` most recently visited solutions instead of
    move ranks (variant R3', PAPER.md:243-244 read literally)."""
    A, S, m, n = _prep(A, S)
    V0 = np.ascontiguousarray(V0, dtype=np.int8)
    tr = np.full(max(iters, 1), -1, dtype=np.int64)
    tf = np.full(max(iters, 1), -1, dtype=np.int64)
    Vo = np.empty(n, dtype=np.int8)
    res = np.zeros(6, dtype=np.int64)
    rc = _load().oracle_tabu_run(_p(A, _i8p), m, n, _p(S, _i32p), k, _p(V0, _i8p), iters,
                                 tenure, int(bool(stop_on_zero)), _p(tr, _i64p),
                                 _p(tf, _i64p), _p(Vo, _i8p), _p(res, _i64p), nthreads,
                                 int(bool(aspiration)) | (2 if tabu_solutions else 0))
    if rc == -2:
        raise ValueError("tenure >= C(n,k): no admissible move would remain")
    if rc != 0:
        raise ValueError("invalid arguments")
    d = dict(zip(RESULT_FIELDS, (int(x) for x in res)))
    it = d["iters_done"]
    return tr[:it].copy(), tf[:it].copy(), Vo, d
