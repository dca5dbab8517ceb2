"""Pins of the CPU oracle against what the paper and mathematics fix (no GPU needed).

Each test names the passage it pins. Nothing here compares the oracle with itself: the
expected values come from hand computation (tests/golden), the paper's worked example and
closed forms, library routines used as *independent* definitions (itertools.combinations is
lexicographic order; sorted() multisets decide f = 0), brute force on tiny inputs, and
invariants that a dropped term, a wrong sign or index, or a transposed operand would break.
"""
import itertools
from math import comb, isqrt

import numpy as np
import pytest

import ppp_inputs as pi
from conftest import golden_lines


# ----------------------------------------------------------------------------- generator
def test_splitmix64_reference_vector(orc):
    want = [int(x, 16) for x in golden_lines("splitmix64_seed0.txt")]
    assert orc.splitmix64(0, 3) == want
    g = pi.splitmix64_stream(0)
    assert [next(g) for _ in range(3)] == want


def test_start_vector_same_on_both_generator_copies(orc):
    for n, seed in [(1, 0), (21, 2), (64, 7), (65, 9), (117, 5), (1024, 6)]:
        assert np.array_equal(orc.start_vector(n, seed), pi.start_vector(n, seed))


@pytest.mark.parametrize("m,n,seed", [(21, 21, 1001), (73, 73, 1002), (16, 16, 3), (20, 17, 4), (64, 64, 5)])
def test_planted_instance_recipe(m, n, seed):
    """north_star recipe: A V* >= 0 after row negation and S = multiset of A V*."""
    I = pi.planted_instance(m, n, seed)
    y = I.A.astype(np.int64) @ I.secret
    assert np.all(y >= 0)
    assert np.array_equal(np.sort(y), np.sort(I.S))
    assert set(np.unique(I.A)) <= {-1, 1}


# ----------------------------------------------------------------------------- rank order
def _paper_pair_rank(n, i, j):
    """Eq. (1): f(i,j) = i(n-1) + (j-1) - i(i+1)/2."""
    return i * (n - 1) + (j - 1) - i * (i + 1) // 2


def _paper_pair_unrank(n, f):
    """Prop. 2 / eqs. (2)-(6), in exact integer arithmetic."""
    m = n * (n - 1) // 2
    X = m - f - 1  # eq. (3)
    k = (isqrt(8 * X + 1) - 1) // 2  # eq. (5)
    i = n - 2 - k  # eq. (2)
    j = f - i * (n - 1) + i * (i + 1) // 2 + 1  # eq. (6)
    return i, j


def _paper_triple_unrank(n, f):
    """Appendix C, exact-integer reading R7: k = ceil(k1) where
    k1^3 - k1 - 6Y = 0 (eq. 9), i.e. the least k with C(k+1,3) >= Y, Y = m - f."""
    m = comb(n, 3)
    Y = m - f
    k = 0
    while comb(k + 1, 3) < Y:
        k += 1
    z = n - k - 1  # eq. (7)
    before = m - (k + 1) * k * (k - 1) // 6  # nbElementsBefore
    nb = k * (k - 1) // 2  # nbElements
    last = before + nb - 1  # lastElement
    fp = f - before  # change of variables
    nprime = n - (z + 1)
    X = last - f
    kk = (isqrt(8 * X + 1) - 1) // 2
    i = nprime - 2 - kk
    j = fp - i * (nprime - 1) + i * (i + 1) // 2 + 1
    return z, i + z + 1, j + z + 1  # x = i + (z+1), y = j + (z+1)


def _paper_triple_rank(n, z, x, y):
    """Appendix D, eqs. (10)-(11), with reading R10 (x in place of y in n3, n4)."""
    k = n - 1 - z
    m = comb(n, 3)
    before = m - (k + 1) * k * (k - 1) // 6
    f1 = z * (n - 2) * (n - 2) + (x - 1) * (n - 2) + (y - 2)
    n1 = z * (n - 2) * (n - 2) - before
    n2 = z * (n - 2)
    n3 = (x - z) * (n - k - 1)
    n4 = (x - z) * (x - z - 1) // 2
    return f1 - n1 - n2 - n3 - n4


def test_paper_worked_example_pair_rank():
    for line in golden_lines("pair_rank_paper.txt"):
        n, i, j, f = map(int, line.split())
        assert _paper_pair_rank(n, i, j) == f
        assert _paper_pair_unrank(n, f) == (i, j)


@pytest.mark.parametrize("k", [1, 2, 3])
@pytest.mark.parametrize("n", [3, 4, 5, 6, 7, 12, 23])
def test_oracle_rank_order_is_lexicographic(orc, n, k):
    """Reading R6: rank = position in lexicographic order (itertools.combinations order)."""
    M = comb(n, k)
    assert orc.neighborhood_size(n, k) == M
    got = orc.flipsets(n, k, np.arange(M))
    want = np.full((M, 3), -1, dtype=np.int32)
    for r, c in enumerate(itertools.combinations(range(n), k)):
        want[r, :k] = c
    assert np.array_equal(got, want)


@pytest.mark.parametrize("n", [3, 4, 6, 9, 17, 40])
def test_paper_index_maps_agree_with_lexicographic_order(n):
    """Props. 1-2 and Appendices A-D define the same order the oracle uses."""
    for r, (i, j) in enumerate(itertools.combinations(range(n), 2)):
        assert _paper_pair_rank(n, i, j) == r
        assert _paper_pair_unrank(n, r) == (i, j)
    for r, (z, x, y) in enumerate(itertools.combinations(range(n), 3)):
        assert _paper_triple_unrank(n, r) == (z, x, y)
        assert _paper_triple_rank(n, z, x, y) == r


def test_neighborhood_sizes_and_paper_caps(orc):
    """PAPER.md:108-125 sizes; Tables I-III caps = C(n,3) (golden/table_caps.txt)."""
    for line in golden_lines("table_caps.txt"):
        n, c1, c2, c3 = map(int, line.split())
        assert (comb(n, 1), comb(n, 2), comb(n, 3)) == (c1, c2, c3)
        if n <= 117:
            assert orc.neighborhood_size(n, 1) == c1
            assert orc.neighborhood_size(n, 2) == c2
            assert orc.neighborhood_size(n, 3) == c3


def test_flipsets_sampled_at_C5_size(orc):
    """Sampled ranks at n = 1024: flip set of rank r equals the r-th lexicographic triple,
    checked by the closed-form lexicographic rank (colex complement, a textbook identity)."""
    n, k = 1024, 3
    M = comb(n, k)
    rng = np.random.default_rng(0)
    ranks = np.unique(np.concatenate([[0, 1, M - 2, M - 1], rng.integers(0, M, 2000)]))
    fs = orc.flipsets(n, k, ranks)
    for r, (a, b, c) in zip(ranks, fs):
        assert 0 <= a < b < c < n
        colex = comb(n - 1 - a, 3) + comb(n - 1 - b, 2) + comb(n - 1 - c, 1)
        assert M - 1 - colex == r


# ----------------------------------------------------------------------------- fitness
def _parse_hand():
    for line in golden_lines("fitness_hand.txt"):
        _, a, s, v, f = [p.strip() for p in line.split("|")]
        A = np.array([[int(x) for x in row.split()] for row in a.split(";")], dtype=np.int8)
        yield A, np.array(s.split(), dtype=np.int32), np.array(v.split(), dtype=np.int8), int(f)


@pytest.mark.parametrize("packed", [False, True])
def test_fitness_hand_computed(orc, packed):
    for A, S, V, f in _parse_hand():
        assert orc.fitness(A, S, V, packed=packed) == f


@pytest.mark.parametrize("m,n,seed", [(21, 21, 1001), (73, 73, 1002), (81, 81, 1003), (101, 117, 1004),
                                      (1024, 1024, 1005), (30, 64, 7), (30, 65, 8), (10, 2, 9)])
def test_planted_secret_has_zero_fitness(orc, m, n, seed):
    """f(V) = 0 is a successful solution; the planted V* is one."""
    I = pi.planted_instance(m, n, seed)
    assert orc.fitness(I.A, I.S, I.secret, packed=True) == 0
    if m * n <= 20000:
        assert orc.fitness(I.A, I.S, I.secret) == 0


@pytest.mark.parametrize("m,n,seed", [(12, 12, 11), (16, 16, 12), (15, 17, 13), (14, 14, 14), (9, 10, 15)])
def test_brute_force_zero_set_is_multiset_equality(orc, m, n, seed):
    """Definition 1 + PAPER.md:238 over all 2^n vectors: f = 0 exactly when
    the multiset {(AV)_j} equals S; f >= 0; f = #negative rows (mod 2)."""
    I = pi.planted_instance(m, n, seed)
    target = np.sort(I.S)
    A64 = I.A.astype(np.int64)
    zeros_oracle, zeros_def = set(), set()
    rng = np.random.default_rng(seed)
    for code in range(1 << n):
        V = np.array([-1 if (code >> i) & 1 else 1 for i in range(n)], dtype=np.int8)
        Y = A64 @ V
        if np.array_equal(np.sort(Y), target):
            zeros_def.add(code)
        # scalar fitness for all vectors would be slow in ctypes; check a random 1/8 plus zeros
        if code in zeros_def or rng.random() < 0.125:
            f = orc.fitness(I.A, I.S, V, packed=True)
            assert f >= 0
            assert f % 2 == int(np.sum(Y < 0)) % 2
            if f == 0:
                zeros_oracle.add(code)
    assert zeros_def  # the planted secret at least
    assert zeros_oracle == zeros_def


def test_fitness_metamorphic_invariants(orc):
    """Row order of A is irrelevant (S is a multiset); permuting / negating columns of A together
    with V is irrelevant; the scalar and popcount paths agree. Catches transposed operands."""
    rng = np.random.default_rng(3)
    for m, n in [(21, 21), (33, 70), (101, 117), (7, 130)]:
        I = pi.planted_instance(m, n, int(rng.integers(1 << 30)))
        for _ in range(5):
            V = np.where(rng.random(n) < 0.5, -1, 1).astype(np.int8)
            f = orc.fitness(I.A, I.S, V)
            assert orc.fitness(I.A, I.S, V, packed=True) == f
            pr, pc = rng.permutation(m), rng.permutation(n)
            assert orc.fitness(I.A[pr], I.S, V) == f
            assert orc.fitness(I.A[:, pc], I.S, V[pc]) == f
            neg = rng.random(n) < 0.5
            A2 = I.A.copy()
            A2[:, neg] *= -1
            V2 = V.copy()
            V2[neg] *= -1
            assert orc.fitness(A2, I.S, V2) == f


def test_penalty_weight_and_histogram_term_separately(orc):
    """With S chosen so the histogram term is known, f isolates 30 * sum(|y| - y)."""
    # one row: A = [1]*n, V = all -1 -> y = -n, S = {n}: f = 30 * 2n + |H_n - 0| = 60 n + 1
    for n in (1, 2, 5, 9):
        A = np.ones((1, n), dtype=np.int8)
        assert orc.fitness(A, np.array([n], np.int32), -np.ones(n, np.int8)) == 60 * n + 1
        # y = n >= 0 but S = {0}: f = |H_0 - 0| + |0 - 1| = 2 (n > 0)
        assert orc.fitness(A, np.array([0], np.int32), np.ones(n, np.int8)) == 2


# ----------------------------------------------------------------------------- neighbourhood
def _flip(V, fs):
    W = V.copy()
    for i in fs:
        if i >= 0:
            W[i] = -W[i]
    return W


@pytest.mark.parametrize("k", [1, 2, 3])
def test_eval_all_matches_scalar_fitness_of_each_neighbour(orc, k):
    """Figs. 7/9/10: new_fitness[rank] = f(V xor F_rank); ranks in itertools order."""
    rng = np.random.default_rng(k)
    I = pi.planted_instance(19, 23, 77)
    V = np.where(rng.random(23) < 0.5, -1, 1).astype(np.int8)
    fa = orc.eval_all(I.A, I.S, V, k)
    assert len(fa) == comb(23, k)
    for r, fs in enumerate(itertools.combinations(range(23), k)):
        assert fa[r] == orc.fitness(I.A, I.S, _flip(V, fs))
    ranks = np.unique(rng.integers(0, len(fa), 50))
    assert np.array_equal(orc.eval_ranks(I.A, I.S, V, k, ranks), fa[ranks])


@pytest.mark.parametrize("k", [1, 2, 3])
def test_eval_best_is_lowest_rank_argmin_over_admissible(orc, k):
    """Reading R5 (lowest rank wins ties) and R3 (tabu ranks are skipped)."""
    rng = np.random.default_rng(10 + k)
    I = pi.planted_instance(15, 18, 5)
    A = I.A.copy()
    A[:, 5] = A[:, 4]  # duplicate columns force ties
    for frac in (0.0, 0.5, 0.9):
        V = np.where(rng.random(18) < 0.5, -1, 1).astype(np.int8)
        fa = orc.eval_all(A, I.S, V, k)
        tabu = rng.random(len(fa)) < frac
        f, r = orc.eval_best(A, I.S, V, k, tabu)
        masked = np.where(tabu, np.iinfo(np.int64).max, fa)
        assert (f, r) == (int(masked.min()), int(np.argmin(masked)))


# ----------------------------------------------------------------------------- tabu search
def _check_tabu_trace(orc, A, S, k, V0, L, tr, tf, res, stop_on_zero, aspiration=False):
    """Each iteration: the accepted rank is the lowest-rank argmin over ranks not accepted in the
    previous L iterations (FIFO tabu list, reading R3, no aspiration R4) -- or, with aspiration,
    over those plus the tabu ranks whose fitness beats the best seen so far (variant R4')."""
    V = V0.copy()
    f = orc.fitness(A, S, V)
    best = f
    n = A.shape[1]
    for t in range(len(tr)):
        assert not (stop_on_zero and f == 0)
        fa = orc.eval_all(A, S, V, k)
        tabu = np.zeros(len(fa), bool)
        tabu[tr[max(0, t - L):t]] = True
        if aspiration:
            tabu &= ~(fa < best)
        masked = np.where(tabu, np.iinfo(np.int64).max, fa)
        assert tr[t] == int(np.argmin(masked)), t
        assert tf[t] == fa[tr[t]]
        (fs,) = orc.flipsets(n, k, [tr[t]])
        V = _flip(V, fs)
        f = int(tf[t])
        best = min(best, f)
        assert orc.fitness(A, S, V) == f
    assert res["final_f"] == f and res["best_f"] == best
    assert res["iters_done"] == len(tr)
    return V


@pytest.mark.parametrize("k,L", [(1, 3), (1, 0), (2, 20), (3, 0), (3, 100)])
def test_tabu_trajectory_rules(orc, k, L):
    I = pi.planted_instance(17, 19, 300 + k)
    V0 = pi.start_vector(19, 4 + k)
    tr, tf, Vo, res = orc.tabu_run(I.A, I.S, k, V0, 40, L, stop_on_zero=False)
    V = _check_tabu_trace(orc, I.A, I.S, k, V0, L, tr, tf, res, False)
    assert np.array_equal(V, Vo)
    if L > 0:  # no rank re-accepted while tabu
        for t in range(len(tr)):
            assert tr[t] not in set(tr[max(0, t - L):t])


def test_tabu_stop_on_zero_reaches_a_solution(orc):
    """C1 shape (21 x 21, k = 1, L = 3): the run that reaches f = 0 stops there and its vector
    reproduces the multiset S (Definition 1), checked with sorted() not with the oracle."""
    I = pi.config_instance("C1")
    solved = 0
    for seed in range(1, 9):
        V0 = pi.start_vector(21, seed)
        tr, tf, Vo, res = orc.tabu_run(I.A, I.S, 1, V0, 1000, 3, stop_on_zero=True)
        _check_tabu_trace(orc, I.A, I.S, 1, V0, 3, tr[:60], tf[:60], {**res, "iters_done": min(60, len(tr)),
                          "final_f": int(tf[min(60, len(tr)) - 1]) if len(tr) else res["final_f"],
                          "best_f": min([orc.fitness(I.A, I.S, V0)] + list(tf[:60]))}, True)
        if res["solved"]:
            solved += 1
            assert res["final_f"] == 0 and res["first_zero_iter"] == res["iters_done"]
            assert np.array_equal(np.sort(I.A.astype(np.int64) @ Vo), np.sort(I.S))
        else:
            assert res["iters_done"] == 1000
    assert solved >= 1


def test_tabu_rejects_tenure_that_exhausts_neighbourhood(orc):
    I = pi.planted_instance(5, 6, 1)
    with pytest.raises(ValueError):
        orc.tabu_run(I.A, I.S, 1, np.ones(6, np.int8), 5, 6)


@pytest.mark.parametrize("k,L", [(1, 5), (2, 60), (3, 300)])
def test_tabu_aspiration_variant(orc, k, L):
    """Aspiration (Taillard [11], variant R4'): a tabu move is allowed when it is better than the
    best fitness found so far; the check re-derives every step by brute force."""
    I = pi.planted_instance(17, 19, 900 + k)
    V0 = pi.start_vector(19, 40 + k)
    tr, tf, Vo, res = orc.tabu_run(I.A, I.S, k, V0, 50, L, stop_on_zero=False, aspiration=True)
    V = _check_tabu_trace(orc, I.A, I.S, k, V0, L, tr, tf, res, False, aspiration=True)
    assert np.array_equal(V, Vo)


def _check_solution_tabu_trace(orc, A, S, k, V0, L, tr, tf, res, aspiration=False):
    """Variant R3' (PAPER.md:243-244 read literally: "the tabu list contains the solutions ...
    visited in the recent past"): at iteration t a neighbour is tabu iff its vector equals one of
    the L most recently visited solutions V_{t-L} .. V_{t-1} (V_0 = the start). Re-derived here by
    brute force on explicit +-1 vectors, not through the oracle's hash set."""
    n = A.shape[1]
    visited = [tuple(int(x) for x in V0)]
    V = V0.copy()
    best = orc.fitness(A, S, V)
    flips = list(itertools.combinations(range(n), k))
    for t in range(len(tr)):
        recent = set(visited[max(0, len(visited) - L):])
        fa = orc.eval_all(A, S, V, k)
        tabu = np.array([tuple(int(x) for x in _flip(V, fs)) in recent for fs in flips])
        if aspiration:
            tabu &= ~(fa < best)
        masked = np.where(tabu, np.iinfo(np.int64).max, fa)
        assert tr[t] == int(np.argmin(masked)), t
        assert tf[t] == fa[tr[t]]
        V = _flip(V, flips[tr[t]])
        visited.append(tuple(int(x) for x in V))
        best = min(best, int(tf[t]))
    assert res["iters_done"] == len(tr) and res["best_f"] == best
    return V


@pytest.mark.parametrize("k,L,aspiration", [(1, 3, False), (1, 8, False), (2, 25, False), (3, 40, False),
                                            (2, 25, True), (1, 1, False)])
def test_tabu_solution_list_variant(orc, k, L, aspiration):
    I = pi.planted_instance(15, 16, 1200 + k + L)
    V0 = pi.start_vector(16, 70 + k)
    tr, tf, Vo, res = orc.tabu_run(I.A, I.S, k, V0, 45, L, stop_on_zero=False, aspiration=aspiration,
                                   tabu_solutions=True)
    V = _check_solution_tabu_trace(orc, I.A, I.S, k, V0, L, tr, tf, res, aspiration)
    assert np.array_equal(V, Vo)
    if not aspiration and L > 1:  # no solution revisited while listed
        seen = [tuple(V0)]
        Vc = V0.copy()
        for t in range(len(tr)):
            (fs,) = orc.flipsets(16, k, [tr[t]])
            Vc = _flip(Vc, fs)
            assert tuple(Vc) not in set(seen[max(0, len(seen) - L):])
            seen.append(tuple(Vc))


# ---------------------------------------------------------------- k > 3
@pytest.mark.parametrize("k", [4, 5, 6, 7])
@pytest.mark.parametrize("n", [7, 8, 11, 16])
def test_oracle_rank_order_k_above_3_is_lexicographic(orc, n, k):
    """k >= 4: the odometer (nested loops generalised) enumerates flip sets in
    itertools.combinations order and counts C(n, k) of them."""
    if k > n:
        return
    M = comb(n, k)
    assert orc.neighborhood_size(n, k) == M
    got = orc.flipsets(n, k, np.arange(M))
    assert np.array_equal(got, np.array(list(itertools.combinations(range(n), k)), dtype=np.int32))


@pytest.mark.parametrize("k", [4, 5])
def test_eval_all_k_above_3_matches_scalar_fitness(orc, k):
    """new_fitness[rank] = f(V xor F_rank) for k = 4, 5 (scalar int8 fitness of the explicitly
    flipped vector, ranks in itertools order), and the sampled / best variants agree."""
    rng = np.random.default_rng(40 + k)
    I = pi.planted_instance(13, 15, 91 + k)
    V = np.where(rng.random(15) < 0.5, -1, 1).astype(np.int8)
    fa = orc.eval_all(I.A, I.S, V, k)
    assert len(fa) == comb(15, k)
    for r, fs in enumerate(itertools.combinations(range(15), k)):
        assert fa[r] == orc.fitness(I.A, I.S, _flip(V, fs))
    ranks = np.unique(rng.integers(0, len(fa), 40))
    assert np.array_equal(orc.eval_ranks(I.A, I.S, V, k, ranks), fa[ranks])
    tabu = rng.random(len(fa)) < 0.3
    bf, br = orc.eval_best(I.A, I.S, V, k, tabu)
    masked = np.where(tabu, np.iinfo(np.int64).max, fa)
    assert br == int(np.argmin(masked)) and bf == fa[br]


@pytest.mark.parametrize("k,L", [(4, 0), (4, 30), (5, 100)])
def test_tabu_trajectory_rules_k_above_3(orc, k, L):
    I = pi.planted_instance(14, 16, 700 + k)
    V0 = pi.start_vector(16, 9 + k)
    tr, tf, Vo, res = orc.tabu_run(I.A, I.S, k, V0, 25, L, stop_on_zero=False)
    V = _check_tabu_trace(orc, I.A, I.S, k, V0, L, tr, tf, res, False)
    assert np.array_equal(V, Vo)
