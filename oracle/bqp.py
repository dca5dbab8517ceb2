"""CPU oracle for the k-Hamming tabu search on a second binary fitness -- TEST INFRASTRUCTURE ONLY.

Only ``tests/``, ``__graft_entry__.smoke()`` and ``bench.py``'s baseline legs may import this
module. It shares no code with the CUDA path and never imports ``paper_conf_ipps_luongmt10_b200``.

Why a second fitness: the paper designs its neighbourhood-to-GPU mappings "for binary problems"
in general (Section I; Section VI) and validates them on one
application, the PPP.
SURVEY.md §8(f) row f4 asks for "a pluggable binary fitness". The fitness chosen here is the
unconstrained binary quadratic programme (UBQP), the textbook generic binary objective:

    minimise  f(x) = x^T Q x = sum_i sum_j Q_ij x_i x_j,   x in {0,1}^n,  Q symmetric int.

Everything else is the paper's search, restated exactly as for the PPP oracle:
  * neighbourhood: every flip set F of k distinct positions, k in {1,2,3},
    ranks in lexicographic order of the sorted flip set (reading R6) -- here
    ``itertools.combinations(range(n), k)``, whose order is exactly that;
  * fitness of a neighbour: f(x xor F) from the definition above (no incremental formula);
  * tabu list: literal until[] array, a rank accepted at iteration t is tabu for t+1..t+L
    (reading R3), default L = floor(C(n,k)/6);
  * selection: least fitness among admissible neighbours, lowest rank on ties (reading R5);
    no aspiration (reading R4); run exactly `iters` iterations (no known target value).

Instances come from ``ppp_inputs.bqp`` (seeded generators only).

Pins (tests/test_bqp_oracle.py, ``-m "not gpu"``): the max-cut identity (f = -cut(x) counted
edge by edge), the closed-form optimum of a planted Ising instance (brute force over all 2^n),
the hand-derived k-flip delta formula, the diagonal special case (closed-form greedy trajectory),
and the tabu invariants (no accepted rank re-enters within L iterations; every accepted move is
the least admissible one).
"""
from __future__ import annotations

from itertools import combinations
from math import comb

import numpy as np


def fitness(Q, x) -> int:
    """f(x) = x^T Q x (definition), exact in int64."""
    Q = np.asarray(Q, dtype=np.int64)
    x = np.asarray(x, dtype=np.int64)
    return int(x @ Q @ x)


def neighborhood_size(n: int, k: int) -> int:
    return comb(n, k)


def flipsets(n: int, k: int) -> np.ndarray:
    """All flip sets in rank order (rank = row index): lexicographic over sorted index tuples."""
    if n < k:
        return np.zeros((0, k), dtype=np.int64)
    return np.array(list(combinations(range(n), k)), dtype=np.int64).reshape(-1, k)


def eval_all(Q, x, k: int) -> np.ndarray:
    """f(x xor F_r) for every rank r, each from the definition x'^T Q x'."""
    Q = np.asarray(Q, dtype=np.int64)
    x = np.asarray(x, dtype=np.int64)
    n = len(x)
    F = flipsets(n, k)
    Xp = np.repeat(x[None, :], len(F), axis=0)
    rows = np.arange(len(F))[:, None]
    Xp[rows, F] ^= 1
    return np.sum((Xp @ Q) * Xp, axis=1)  # row r: x_r'^T Q x_r'


def tabu_run(Q, x0, k: int, iters: int, tenure: int = -1):
    """The tabu search of PAPER.md:241-258 on f(x) = x^T Q x.

    Returns (trace_rank, trace_fit, x_out, result) with result = dict(iters_done, final_f,
    best_f, best_iter). tenure < 0 selects floor(C(n,k)/6). Raises ValueError when every
    neighbour is tabu (only possible for tenure >= C(n,k), which is rejected up front)."""
    Q = np.asarray(Q, dtype=np.int64)
    x = np.array(x0, dtype=np.int64)
    n = len(x)
    M = comb(n, k)
    L = M // 6 if tenure < 0 else tenure
    if L >= M:
        raise ValueError("tenure >= C(n,k): no admissible move would remain")
    F = flipsets(n, k)
    until = np.zeros(M, dtype=np.int64)  # admissible at t iff until[r] < t
    f = fitness(Q, x)
    best_f, best_iter = f, 0
    tr, tf = [], []
    for t in range(1, iters + 1):
        fits = eval_all(Q, x, k)
        adm = until < t
        cand = np.where(adm, fits, np.iinfo(np.int64).max)
        r = int(np.argmin(cand))  # first minimum: lowest rank on ties (reading R5)
        assert adm[r]
        x[F[r]] ^= 1
        f = int(fits[r])
        until[r] = t + L
        tr.append(r)
        tf.append(f)
        if f < best_f:
            best_f, best_iter = f, t
    res = dict(iters_done=iters, final_f=f, best_f=best_f, best_iter=best_iter)
    return np.array(tr, dtype=np.int64), np.array(tf, dtype=np.int64), x.astype(np.uint8), res

