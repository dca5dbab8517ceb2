"""Pins of the UBQP oracle (oracle/bqp.py) against what the mathematics fixes -- CPU only.

Each pin is independent of the definition the oracle writes out (f = x^T Q x, neighbours by
itertools.combinations), so a dropped term, a wrong sign or index, or a wrong rank order fails
one of them. DESIGN.md §5.13.
"""
from itertools import product
from math import comb

import numpy as np
import pytest

from oracle import bqp
from ppp_inputs import bqp as bi


def _cut(W, x):
    """Weight of the edges crossing (x = 0 | x = 1), counted edge by edge."""
    n = len(x)
    return sum(int(W[i][j]) for i in range(n) for j in range(i + 1, n) if x[i] != x[j])


def test_fitness_is_minus_maxcut():
    """Textbook reduction: with Q = W - diag(W 1), x^T Q x = -cut(x) for every x."""
    rng = np.random.default_rng(5)
    n = 9
    W = np.triu(rng.integers(0, 10, size=(n, n)), 1)
    W = W + W.T
    Q = W - np.diag(W.sum(axis=1))
    for bits in product((0, 1), repeat=n):
        x = np.array(bits)
        assert bqp.fitness(Q, x) == -_cut(W, x)


@pytest.mark.parametrize("n,seed", [(8, 1), (11, 2), (12, 3)])
def test_planted_ising_closed_form_optimum(n, seed):
    """min over all 2^n x of x^T Q x equals -n^2 - 1^T J 1 = -n^2 + (sum z)^2, attained exactly
    at x = (1 + z)/2 and its complement (s = 2x - 1 = +-z)."""
    Q, z = bi.planted_ising(n, seed)
    fmin = -n * n + int(z.sum()) ** 2
    xs = np.array(list(product((0, 1), repeat=n)), dtype=np.int64)
    f = np.einsum("ri,ij,rj->r", xs, Q.astype(np.int64), xs)
    assert f.min() == fmin
    arg = {tuple(r) for r in xs[f == fmin]}
    xz = tuple(((1 + z) // 2).tolist())
    assert arg == {xz, tuple(1 - np.array(xz))}
    assert bqp.fitness(Q, np.array(xz)) == fmin


@pytest.mark.parametrize("k", [1, 2, 3])
def test_eval_all_matches_flip_delta(k):
    """Hand derivation: x' = x + d on F (d_i = 1 - 2 x_i), Q symmetric ->
    f(x') - f(x) = sum_{i in F} (2 d_i g_i + Q_ii) + 2 sum_{i<j in F} d_i d_j Q_ij, g = Q x."""
    n = 13
    Q = bi.random_q(n, 0.6, 7).astype(np.int64)
    x = bi.start_x(n, 3).astype(np.int64)
    g = Q @ x
    f0 = int(x @ Q @ x)
    got = bqp.eval_all(Q, x, k)
    exp = []
    for F in bqp.flipsets(n, k):
        d = {i: 1 - 2 * int(x[i]) for i in F}
        delta = sum(2 * d[i] * int(g[i]) + int(Q[i, i]) for i in F)
        delta += 2 * sum(d[i] * d[j] * int(Q[i, j]) for a, i in enumerate(F) for j in F[a + 1:])
        exp.append(f0 + delta)
    assert got.tolist() == exp


def test_rank_order_is_lexicographic():
    """Rank order = lexicographic order of the sorted flip set (reading R6): first/last ranks and
    the worked example of PAPER.md:473-474 (Appendix A, Fig. 11: n = 6, m = 15, the neighbour
    (i = 2, j = 3) has 1D index f(i, j) = 9)."""
    F = bqp.flipsets(6, 2)
    assert len(F) == comb(6, 2)
    assert F[0].tolist() == [0, 1] and F[-1].tolist() == [4, 5]
    assert F[9].tolist() == [2, 3]
    F3 = bqp.flipsets(7, 3)
    assert all(tuple(F3[i]) < tuple(F3[i + 1]) for i in range(len(F3) - 1))


def test_diagonal_greedy_trajectory():
    """Q = diag(c), x0 = 0, k = 1, tenure 0: each move takes the most negative remaining c_i
    (closed form: f drops by c_i); once every negative c is set the search oscillates on the
    least |c| move. Trajectory from the closed form."""
    c = np.array([5, -3, -9, 0, -1, 7, -4])
    Q = np.diag(c)
    tr, tf, xo, res = bqp.tabu_run(Q, np.zeros(7, dtype=np.uint8), 1, 6, tenure=0)
    assert tr.tolist()[:4] == [2, 6, 1, 4]
    assert tf.tolist()[:4] == [-9, -13, -16, -17]
    assert res["best_f"] == int(c[c < 0].sum()) == -17
    # step 5: every move is uphill; the cheapest is flipping c = 0 (index 3) -> f stays -17
    assert tr[4] == 3 and tf[4] == -17


@pytest.mark.parametrize("k,tenure", [(1, 3), (2, -1), (3, 20)])
def test_tabu_invariants(k, tenure):
    """Every accepted move is the least-fitness, lowest-rank admissible neighbour of the current
    x (recomputed here by brute force from x), and no rank is accepted twice within L iterations."""
    n = 10
    Q = bi.random_q(n, 0.5, 11)
    x0 = bi.start_x(n, 4)
    iters = 40
    tr, tf, xo, res = bqp.tabu_run(Q, x0, k, iters, tenure)
    M = comb(n, k)
    L = M // 6 if tenure < 0 else tenure
    F = list(__import__("itertools").combinations(range(n), k))
    x = x0.astype(np.int64).copy()
    last = {}
    for t in range(1, iters + 1):
        best = None
        for r, fs in enumerate(F):
            if r in last and t <= last[r] + L:
                continue
            y = x.copy()
            y[list(fs)] ^= 1
            fy = int(y @ Q.astype(np.int64) @ y)
            if best is None or fy < best[0]:
                best = (fy, r)
        assert (int(tf[t - 1]), int(tr[t - 1])) == best
        x[list(F[best[1]])] ^= 1
        last[best[1]] = t
    assert xo.tolist() == x.tolist()
    assert res["best_f"] == min([bqp.fitness(Q, x0)] + tf.tolist())


def test_tenure_too_large_rejected():
    with pytest.raises(ValueError):
        bqp.tabu_run(np.eye(4, dtype=np.int64), np.zeros(4), 1, 3, tenure=4)
