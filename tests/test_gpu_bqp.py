"""GPU parity of the second binary fitness (UBQP): the CUDA path through the C ABI
against oracle/bqp.py, element by element. Integer arithmetic: every comparison is exact."""
from math import comb

import numpy as np
import pytest

from oracle import bqp
from ppp_inputs import bqp as bi

pytestmark = pytest.mark.gpu


@pytest.fixture(scope="module")
def L():
    import torch

    if not torch.cuda.is_available():
        pytest.skip("no CUDA device")
    import paper_conf_ipps_luongmt10_b200 as lib

    lib.load()
    return lib


def _states(n, seed):
    return [bi.start_x(n, seed), np.zeros(n, np.uint8), np.ones(n, np.uint8), bi.start_x(n, seed + 1)]


def _lex_unrank(n, k, r):
    """Test-side lexicographic unranking (walks the first index up, counting the sets it skips)."""
    out, lo = [], 0
    for q in range(k, 0, -1):
        i = lo
        while comb(n - 1 - i, q - 1) <= r:
            r -= comb(n - 1 - i, q - 1)
            i += 1
        out.append(i)
        lo = i + 1
    return out


@pytest.mark.parametrize("k,n,dens", [(1, 1, 1.0), (1, 97, 0.3), (1, 400, 0.1), (2, 2, 1.0), (2, 13, 0.6),
                                      (2, 97, 0.2), (2, 200, 0.1), (3, 3, 1.0), (3, 20, 0.5), (3, 61, 0.3),
                                      (3, 70, 0.1)])
def test_eval_all_matches_oracle(L, k, n, dens):
    Q = bi.random_q(n, dens, 100 + n + k)
    ctx = L.lns_bqp_create(Q, 0)
    try:
        for x in _states(n, 7 * n + k):
            got = L.lns_bqp_eval_all(ctx, k, x).astype(np.int64)
            assert np.array_equal(got, bqp.eval_all(Q, x, k))
    finally:
        L.lns_bqp_destroy(ctx)


@pytest.mark.parametrize("k", [1, 2, 3])
def test_eval_all_planted_ising(L, k):
    n = 33
    Q, z = bi.planted_ising(n, 9 + k)
    ctx = L.lns_bqp_create(Q, 0)
    try:
        for x in _states(n, k) + [((1 + z) // 2).astype(np.uint8)]:
            assert np.array_equal(L.lns_bqp_eval_all(ctx, k, x).astype(np.int64), bqp.eval_all(Q, x, k))
    finally:
        L.lns_bqp_destroy(ctx)


@pytest.mark.parametrize("k,n", [(2, 1500), (3, 300)])
def test_eval_all_large_sampled(L, k, n):
    """Sizes past the oracle's einsum: 300 sampled ranks (incl. first / last) from the definition."""
    Q = bi.random_q(n, 0.05, 3 + k)
    x = bi.start_x(n, 5)
    ctx = L.lns_bqp_create(Q, 0)
    try:
        got = L.lns_bqp_eval_all(ctx, k, x)
    finally:
        L.lns_bqp_destroy(ctx)
    M = comb(n, k)
    assert len(got) == M
    rng = np.random.default_rng(1)
    for r in [0, 1, M - 2, M - 1] + rng.integers(0, M, 296).tolist():
        y = x.copy()
        y[_lex_unrank(n, k, int(r))] ^= 1
        assert int(got[r]) == bqp.fitness(Q, y), r


@pytest.mark.parametrize("k,n,iters,tenure", [(1, 30, 300, -1), (1, 30, 200, 0), (2, 25, 200, -1),
                                              (2, 25, 130, 7), (3, 20, 150, 50), (3, 16, 64, -1), (3, 16, 5, 0)])
def test_tabu_trajectory_bit_exact(L, k, n, iters, tenure):
    """Whole trajectories (graph-replayed blocks of 64 iterations + remainder) against the oracle."""
    Q = bi.random_q(n, 0.4, 50 + k)
    x0 = bi.start_x(n, 11)
    ctx = L.lns_bqp_create(Q, 0)
    try:
        tr, tf, xo, res = L.lns_bqp_tabu_run(ctx, k, iters, tenure, x0)
    finally:
        L.lns_bqp_destroy(ctx)
    otr, otf, oxo, ores = bqp.tabu_run(Q, x0, k, iters, tenure)
    assert res == ores
    assert np.array_equal(tr, otr) and np.array_equal(tf, otf) and np.array_equal(xo, oxo)


@pytest.mark.parametrize("k", [1, 2, 3])
def test_positive_and_mixed_sign_fitnesses(L, k):
    """Q >= 0 from x = 0: every neighbour has f > 0 (the key's biased high word above 2^31), then
    trajectories that cross from positive to negative fitness: keys order correctly across the
    sign boundary."""
    n = 24
    Q = np.abs(bi.random_q(n, 0.5, 21 + k)) + np.eye(n, dtype=np.int32)
    x0 = np.zeros(n, np.uint8)
    ctx = L.lns_bqp_create(Q, 0)
    try:
        got = L.lns_bqp_eval_all(ctx, k, x0).astype(np.int64)
        assert got.min() > 0 and np.array_equal(got, bqp.eval_all(Q, x0, k))
        tr, tf, xo, res = L.lns_bqp_tabu_run(ctx, k, 70, -1, x0)
        otr, otf, oxo, ores = bqp.tabu_run(Q, x0, k, 70, -1)
        assert res == ores and np.array_equal(tr, otr) and np.array_equal(tf, otf)
    finally:
        L.lns_bqp_destroy(ctx)
    Q2 = bi.random_q(n, 0.5, 31 + k) + 60 * np.eye(n, dtype=np.int32)  # mixed signs around 0
    ctx = L.lns_bqp_create(Q2, 0)
    try:
        for x in _states(n, 3):
            tr, tf, xo, res = L.lns_bqp_tabu_run(ctx, k, 80, -1, x)
            otr, otf, oxo, ores = bqp.tabu_run(Q2, x, k, 80, -1)
            assert res == ores and np.array_equal(tr, otr) and np.array_equal(tf, otf)
    finally:
        L.lns_bqp_destroy(ctx)


def test_tabu_reaches_planted_optimum(L):
    """Planted Ising (closed-form optimum -n^2 + (sum z)^2): k = 2 from a random x;
    same trajectory as the oracle, and the optimum is reached."""
    n = 40
    Q, z = bi.planted_ising(n, 77)
    x0 = bi.start_x(n, 78)
    ctx = L.lns_bqp_create(Q, 0)
    try:
        tr, tf, xo, res = L.lns_bqp_tabu_run(ctx, 2, 60, -1, x0)
    finally:
        L.lns_bqp_destroy(ctx)
    otr, otf, oxo, ores = bqp.tabu_run(Q, x0, 2, 60, -1)
    assert res == ores and np.array_equal(tr, otr)
    assert res["best_f"] == -n * n + int(z.sum()) ** 2


def test_device_buffers_and_untraced(L):
    import torch

    n, k = 50, 2
    Q = bi.random_q(n, 0.3, 4)
    x0 = bi.start_x(n, 2)
    ctx = L.lns_bqp_create(torch.from_numpy(Q).cuda(), 0)
    try:
        out = torch.empty(comb(n, k), dtype=torch.int32, device="cuda")
        L.lns_bqp_eval_all(ctx, k, torch.from_numpy(x0).cuda(), out=out)
        assert np.array_equal(out.cpu().numpy().astype(np.int64), bqp.eval_all(Q, x0, k))
        xo = torch.empty(n, dtype=torch.uint8, device="cuda")
        tr, tf, _, res = L.lns_bqp_tabu_run(ctx, k, 100, -1, torch.from_numpy(x0).cuda(), x_out=xo, trace=False)
        assert tr is None
        _, _, oxo, ores = bqp.tabu_run(Q, x0, k, 100, -1)
        assert res == ores and np.array_equal(xo.cpu().numpy(), oxo)
        assert L.lns_bqp_last_kernel_ms(ctx) > 0
    finally:
        L.lns_bqp_destroy(ctx)


def test_errors(L):
    Q = bi.random_q(8, 0.5, 1)
    bad = Q.copy()
    bad[0, 1] += 1
    with pytest.raises(L.LnsError) as e:
        L.lns_bqp_create(bad, 0)
    assert e.value.status == L.LNS_EINVAL
    with pytest.raises(L.LnsError) as e:
        L.lns_bqp_create(np.full((4, 4), 1 << 26, np.int32), 0)
    assert e.value.status == L.LNS_ERANGE
    ctx = L.lns_bqp_create(Q, 0)
    try:
        x = np.zeros(8, np.uint8)
        for k in (0, 4):
            with pytest.raises(L.LnsError) as e:
                L.lns_bqp_eval_all(ctx, k, x, out=np.empty(100, np.int32))
            assert e.value.status == L.LNS_EINVAL
        x2 = x.copy()
        x2[3] = 2
        with pytest.raises(L.LnsError) as e:
            L.lns_bqp_eval_all(ctx, 1, x2)
        assert e.value.status == L.LNS_EINVAL
        with pytest.raises(L.LnsError) as e:
            L.lns_bqp_tabu_run(ctx, 1, 5, 8, x)
        assert e.value.status == L.LNS_ERANGE
        # still usable after the errors
        assert np.array_equal(L.lns_bqp_eval_all(ctx, 1, x).astype(np.int64), bqp.eval_all(Q, x, 1))
    finally:
        L.lns_bqp_destroy(ctx)
    tiny = L.lns_bqp_create(np.array([[3, -1], [-1, 2]], np.int32), 0)
    try:
        with pytest.raises(L.LnsError) as e:
            L.lns_bqp_eval_all(tiny, 3, np.zeros(2, np.uint8), out=np.empty(1, np.int32))
        assert e.value.status == L.LNS_EINVAL
    finally:
        L.lns_bqp_destroy(tiny)


@pytest.mark.parametrize("k,n,R,iters,tenure", [(1, 40, 7, 150, -1), (2, 33, 5, 130, 9), (2, 25, 1, 70, -1),
                                                (3, 22, 12, 140, -1), (3, 18, 33, 40, 0), (3, 60, 4, 200, 300)])
def test_batched_restarts_bit_exact(L, k, n, R, iters, tenure):
    """lns_bqp_tabu_run_batch: every restart (one grid row each, graph blocks + remainder) ends where
    the oracle's search from the same start ends: result fields and final x, restart by restart."""
    Q = bi.random_q(n, 0.35, 70 + k + n)
    X0 = np.stack([bi.start_x(n, 100 + r) for r in range(R)])
    ctx = L.lns_bqp_create(Q, 0)
    try:
        Xo = np.empty_like(X0)
        res = L.lns_bqp_tabu_run_batch(ctx, k, X0, iters, tenure, x_outs=Xo)
        # the context's single-search state is untouched by a batch (and vice versa)
        _, _, xo1, res1 = L.lns_bqp_tabu_run(ctx, k, iters, tenure, X0[R - 1])
    finally:
        L.lns_bqp_destroy(ctx)
    for r in range(R):
        _, _, oxo, ores = bqp.tabu_run(Q, X0[r], k, iters, tenure)
        assert res[r] == ores, r
        assert np.array_equal(Xo[r], oxo), r
    assert res1 == res[R - 1] and np.array_equal(xo1, Xo[R - 1])


def test_batched_restarts_device_buffers_and_errors(L):
    import torch

    n, k, R = 30, 3, 6
    Q = bi.random_q(n, 0.3, 9)
    X0 = np.stack([bi.start_x(n, 7 + r) for r in range(R)])
    ctx = L.lns_bqp_create(Q, 0)
    try:
        Xo = torch.empty((R, n), dtype=torch.uint8, device="cuda")
        res = L.lns_bqp_tabu_run_batch(ctx, k, torch.from_numpy(X0).cuda(), 90, -1, x_outs=Xo)
        for r in (0, R - 1):
            _, _, oxo, ores = bqp.tabu_run(Q, X0[r], k, 90, -1)
            assert res[r] == ores and np.array_equal(Xo[r].cpu().numpy(), oxo)
        bad = X0.copy()
        bad[2, 5] = 3
        with pytest.raises(L.LnsError) as e:
            L.lns_bqp_tabu_run_batch(ctx, k, bad, 10)
        assert e.value.status == L.LNS_EINVAL
        with pytest.raises(L.LnsError) as e:
            L.lns_bqp_tabu_run_batch(ctx, k, X0, 10, comb(n, k))
        assert e.value.status == L.LNS_ERANGE
        with pytest.raises(L.LnsError) as e:
            L.lns_bqp_tabu_run_batch(ctx, k, X0[:0], 10)
        assert e.value.status == L.LNS_EINVAL
    finally:
        L.lns_bqp_destroy(ctx)
