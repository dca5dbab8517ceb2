"""GPU parity: the CUDA path (through the C ABI) against the CPU oracle, element by element.

All work is integer, so every comparison is exact (bit-exact fitness values, ranks and whole
trajectories). Inputs are the seeded planted instances of ppp_inputs.
"""
import os
from math import comb

import numpy as np
import pytest

import ppp_inputs as pi

pytestmark = pytest.mark.gpu


@pytest.fixture(scope="module")
def L():
    import torch

    if not torch.cuda.is_available():
        pytest.skip("no CUDA device")
    import paper_conf_ipps_luongmt10_b200 as lib

    lib.load()
    return lib


def _rand_pm1(rng, n):
    return np.where(rng.random(n) < 0.5, -1, 1).astype(np.int8)


def _states(inst, rng, count=3):
    """Random V, near-solution V (secret with 1-3 flips), and V = -secret (every row negative)."""
    n = inst.n
    out = [_rand_pm1(rng, n) for _ in range(count)]
    near = inst.secret.copy()
    near[rng.choice(n, size=min(3, n), replace=False)] *= -1
    out.append(near)
    out.append((-inst.secret).astype(np.int8))
    out.append(inst.secret.copy())
    return out


# ------------------------------------------------------------------------------ unranking
@pytest.mark.parametrize("k", [1, 2, 3])
def test_unrank_exhaustive_small(L, orc, k):
    for n in (3, 4, 5, 7, 31, 32, 33, 60):
        M = comb(n, k)
        r = np.arange(M, dtype=np.int64)
        assert np.array_equal(L.lns_unrank(n, k, r), orc.flipsets(n, k, r))


def test_unrank_exhaustive_C4(L, orc):
    n, k = 117, 3
    r = np.arange(comb(n, k), dtype=np.int64)
    assert np.array_equal(L.lns_unrank(n, k, r), orc.flipsets(n, k, r))


@pytest.mark.parametrize("n", [1024, 2954])
def test_unrank_sampled_large(L, orc, n):
    """Full-size rank spaces (C5: 1.78e8 ranks; the largest n with C(n,3) < 2^32): random ranks
    plus every plan boundary (first/last rank of each smallest index)."""
    k = 3
    M = comb(n, k)
    rng = np.random.default_rng(n)
    firsts = [0]
    for a in range(n - 3):
        firsts.append(firsts[-1] + comb(n - 1 - a, 2))
    bnd = np.array(firsts, dtype=np.int64)
    ranks = np.unique(np.concatenate([bnd, bnd - 1, bnd + 1, rng.integers(0, M, 200000), [M - 1]]))
    ranks = ranks[(ranks >= 0) & (ranks < M)]
    assert np.array_equal(L.lns_unrank(n, k, ranks), orc.flipsets(n, k, ranks))


# ------------------------------------------------------------------------------ evaluation
SHAPES = [(21, 21, 1), (73, 73, 2), (19, 23, 3), (33, 40, 3), (64, 64, 3), (30, 30, 2), (65, 66, 1),
          (81, 81, 3), (101, 117, 3), (1, 5, 3), (32, 3, 3), (200, 50, 3)]


@pytest.mark.parametrize("m,n,k", SHAPES)
def test_eval_all_matches_oracle(L, orc, m, n, k):
    inst = pi.planted_instance(m, n, 7000 + m * 31 + n)
    rng = np.random.default_rng(m * n + k)
    ctx = L.lns_create(inst.A, inst.S)
    try:
        for V in _states(inst, rng, count=2):
            got = L.lns_eval_all(ctx, k, V)
            want = orc.eval_all(inst.A, inst.S, V, k)
            assert np.array_equal(got.astype(np.int64), want)
    finally:
        L.lns_destroy(ctx)


@pytest.mark.parametrize("m,n,k", [(160, 41, 3), (240, 53, 2), (300, 61, 3), (600, 45, 3)])
def test_deep_rows_table_boundary(L, orc, m, n, k):
    """The deep rows' column table is used from two deep row words on: states whose
    deep-negative rows (Y < -2k, every destination negative) number just below, at and above 32
    and 64 (table off / on) give the oracle's fitness for every neighbour, on the packed path
    (m <= 255) and the m > 255 path."""
    inst = pi.planted_instance(m, n, 9100 + m + n)
    rng = np.random.default_rng(m + k)
    A = inst.A.astype(np.int32)
    want_counts = {31, 32, 33, 63, 64, 65, 97}
    seen = set()
    ctx = L.lns_create(inst.A, inst.S)
    try:
        for trial in range(4000):
            V = (-inst.secret).astype(np.int8)
            flip = rng.choice(n, size=int(rng.integers(1, n)), replace=False)
            V[flip] *= -1
            deep = int(((A @ V.astype(np.int32)) < -2 * k).sum())
            if deep not in want_counts or deep in seen:
                continue
            seen.add(deep)
            got = L.lns_eval_all(ctx, k, V).astype(np.int64)
            assert np.array_equal(got, orc.eval_all(inst.A, inst.S, V, k)), deep
            if len(seen) == len(want_counts):
                break
    finally:
        L.lns_destroy(ctx)
    assert {31, 33}.issubset(seen) or {63, 65}.issubset(seen), seen  # both sides of a threshold


def test_eval_all_forced_ties_duplicate_columns(L, orc):
    inst = pi.planted_instance(40, 30, 99)
    A = inst.A.copy()
    A[:, 7] = A[:, 3]
    A[:, 20] = -A[:, 11]
    ctx = L.lns_create(A, inst.S)
    try:
        rng = np.random.default_rng(1)
        for k in (1, 2, 3):
            V = _rand_pm1(rng, 30)
            assert np.array_equal(L.lns_eval_all(ctx, k, V).astype(np.int64), orc.eval_all(A, inst.S, V, k))
    finally:
        L.lns_destroy(ctx)


@pytest.mark.parametrize("m,n,k", [(21, 21, 1), (73, 73, 2), (81, 81, 3), (101, 117, 3), (47, 33, 3)])
def test_eval_neighborhood_best_with_tabu(L, orc, m, n, k):
    inst = pi.planted_instance(m, n, 4242 + n)
    rng = np.random.default_rng(n)
    M = comb(n, k)
    ctx = L.lns_create(inst.A, inst.S)
    try:
        for V in _states(inst, rng, count=1):
            Y = (inst.A.astype(np.int32) @ V.astype(np.int32)).astype(np.int32)
            for frac in (0.0, 0.5, 1.0):
                tabu = rng.random(M) < frac
                if frac == 1.0:
                    tabu[rng.integers(M)] = False  # exactly one admissible rank
                bits = np.packbits(tabu, bitorder="little")
                bits = np.concatenate([bits, np.zeros((-len(bits)) % 4, np.uint8)]).view(np.uint32)
                got = L.lns_eval_neighborhood(ctx, k, V, Y, bits)
                assert got == orc.eval_best(inst.A, inst.S, V, k, tabu)
    finally:
        L.lns_destroy(ctx)


def test_eval_neighborhood_errors(L):
    inst = pi.planted_instance(21, 21, 1)
    ctx = L.lns_create(inst.A, inst.S)
    try:
        V = inst.secret
        Y = (inst.A.astype(np.int32) @ V).astype(np.int32)
        with pytest.raises(L.LnsError) as e:
            L.lns_eval_neighborhood(ctx, 1, V, Y + 2)
        assert e.value.status == L.LNS_EINVAL
        with pytest.raises(L.LnsError) as e:
            L.lns_eval_neighborhood(ctx, 8, V, Y)  # k in 1..7
        assert e.value.status == L.LNS_EINVAL
        with pytest.raises(L.LnsError) as e:
            L.lns_eval_neighborhood(ctx, 4, V, Y + 2)  # the k > 3 path checks Y = A V too
        assert e.value.status == L.LNS_EINVAL
        allbits = np.full(1, 0xFFFFFFFF, np.uint32)
        with pytest.raises(L.LnsError) as e:
            L.lns_eval_neighborhood(ctx, 1, V, Y, allbits)
        assert e.value.status == L.LNS_ENOADMISSIBLE
        with pytest.raises(L.LnsError) as e:
            L.lns_tabu_run(ctx, 1, 10, tenure=21)
        assert e.value.status == L.LNS_ERANGE
    finally:
        L.lns_destroy(ctx)
    with pytest.raises(L.LnsError) as e:
        L.lns_create(np.zeros((2, 2), np.int8), np.zeros(2, np.int32))
    assert e.value.status == L.LNS_EINVAL
    with pytest.raises(L.LnsError) as e:
        L.lns_create(np.ones((2, 2), np.int8), np.array([0, 3], np.int32))
    assert e.value.status == L.LNS_EINVAL


C5_SAMPLE = 100_000  # >= 1e5 (V, F) per config


@pytest.mark.parametrize("state", ["random", "near_secret", "minus_secret"])
def test_eval_C5_sampled(L, orc, state):
    """C5 (1024 x 1024, k = 3, 1.78e8 neighbours, the launch configuration the bench times): 1e5
    sampled fitnesses (plus every plan-boundary rank of the first and last plans) against the
    oracle's from-scratch fitness, on a random start, a near-solution state (the secret with 3
    flips) and V = -secret (every row negative: the deep-negative shortcut). The returned best
    equals the minimum of the full GPU array and has the oracle's fitness."""
    import torch

    inst = pi.config_instance("C5")
    rng = np.random.default_rng({"random": 5, "near_secret": 6, "minus_secret": 7}[state])
    if state == "random":
        V = pi.start_vector(1024, pi.config_seed("C5"))
    elif state == "near_secret":
        V = inst.secret.copy()
        V[rng.choice(1024, size=3, replace=False)] *= -1
    else:
        V = (-inst.secret).astype(np.int8)
    M = comb(1024, 3)
    ctx = L.lns_create(inst.A, inst.S)
    try:
        out = torch.empty(M, dtype=torch.int32, device="cuda")
        L.lns_eval_all(ctx, 3, V, out)
        edges = [0, 1, 1021, 1022, comb(1023, 2) - 1, comb(1023, 2), M - 2, M - 1]
        ranks = np.unique(np.concatenate([rng.integers(0, M, C5_SAMPLE), edges]))
        got = out[torch.from_numpy(ranks).cuda()].cpu().numpy().astype(np.int64)
        want = orc.eval_ranks(inst.A, inst.S, V, 3, ranks)
        bad = np.nonzero(got != want)[0]
        assert len(bad) == 0, (len(bad), ranks[bad[:5]], got[bad[:5]], want[bad[:5]])
        Y = (inst.A.astype(np.int32) @ V.astype(np.int32)).astype(np.int32)
        bf, br = L.lns_eval_neighborhood(ctx, 3, V, Y)
        mn = int(out.min().item())
        first = int(torch.nonzero(out == mn)[0].item())
        assert (bf, br) == (mn, first)
        assert orc.eval_ranks(inst.A, inst.S, V, 3, [br])[0] == bf
    finally:
        L.lns_destroy(ctx)


def test_C5_trajectory_matches_oracle_golden(L):
    """BASELINE configs[4] (C5): the first iterations of the single-GPU search equal, bit for bit,
    the oracle's trajectory stored in tests/golden/c5_trajectory.txt (written by
    scripts/golden_c5.py from oracle/ only: every one of the 1.78e8 neighbours per iteration
    recomputed from scratch). This checks the C5 argmin against the
    oracle, not against the GPU's own array."""
    from conftest import golden_lines

    rows = list(golden_lines("c5_trajectory.txt"))
    f0 = int(next(r for r in rows if r.startswith("f0 ")).split()[1])
    steps = [tuple(int(x) for x in r.split()) for r in rows if r[0].isdigit()]
    vsha = next(r for r in rows if r.startswith("V_out_sha256 ")).split()[1]
    iters = len(steps)
    assert iters >= 2
    import hashlib

    inst = pi.config_instance("C5")
    seed = pi.config_seed("C5")
    with L.Instance(inst.A, inst.S) as I:
        tr, tf, Vo, res = I.tabu_run(3, iters, -1, seed=seed, stop_on_zero=False)
    assert res["iters_done"] == iters
    assert [(t + 1, int(tr[t]), int(tf[t])) for t in range(iters)] == steps
    assert res["best_f"] == min(f0, min(s[2] for s in steps))
    assert hashlib.sha256(np.ascontiguousarray(Vo, np.int8).tobytes()).hexdigest() == vsha


# ------------------------------------------------------------------------------ trajectories
# SURVEY.md §8(d) parity runs: C1/C2 full, C3 the 10,000-iteration trace, C4 2,000 iterations
TRAJ = [("C1", 1000, True), ("C1", 1000, False), ("C2", 10000, False), ("C3", 10000, False), ("C4", 2000, False)]


@pytest.mark.parametrize("cfg,iters,stop", TRAJ)
def test_tabu_trajectory_bit_exact(L, orc, cfg, iters, stop):
    c = pi.CONFIGS[cfg]
    inst = pi.config_instance(cfg)
    seed = pi.config_seed(cfg)
    V0 = pi.start_vector(inst.n, seed)
    L_ten = pi.default_tenure(inst.n, c["k"])
    with L.Instance(inst.A, inst.S) as I:
        tr, tf, Vo, res = I.tabu_run(c["k"], iters, -1, seed=seed, V0=None, stop_on_zero=stop)
    otr, otf, oVo, ores = orc.tabu_run(inst.A, inst.S, c["k"], V0, iters, L_ten, stop_on_zero=stop)
    assert res == ores
    assert np.array_equal(tr, otr)
    assert np.array_equal(tf, otf)
    assert np.array_equal(Vo, oVo)


@pytest.mark.parametrize("k,L_ten", [(1, 0), (2, 1), (2, 2), (3, 5), (3, 0)])
def test_trajectory_short_tenures_and_forced_stepped(L, orc, k, L_ten):
    """Tenures 0, 1, 2 exercise the ring-buffer edge cases; the stepped launch sequence (the
    multi-GPU code path) must give the same trajectory as the persistent kernel."""
    inst = pi.planted_instance(37, 29, 555 + k)
    V0 = pi.start_vector(29, 11 + k)
    otr, otf, oVo, ores = orc.tabu_run(inst.A, inst.S, k, V0, 150, L_ten, stop_on_zero=False)
    with L.Instance(inst.A, inst.S) as I:
        for flags in (0, L.LNS_FORCE_STEPPED):
            tr, tf, Vo, res = I.tabu_run(k, 150, L_ten, V0=V0, stop_on_zero=False, flags=flags)
            assert res == ores and np.array_equal(tr, otr) and np.array_equal(tf, otf)
            assert np.array_equal(Vo, oVo)


@pytest.mark.parametrize("blocks", [1, 2, 7, 148])
def test_trajectory_independent_of_grid_size(L, orc, blocks):
    inst = pi.config_instance("C3")
    V0 = pi.start_vector(81, 4)
    otr, otf, _, ores = orc.tabu_run(inst.A, inst.S, 3, V0, 60, pi.default_tenure(81, 3), stop_on_zero=False)
    with L.Instance(inst.A, inst.S) as I:
        L.lns_config(I.ctx, blocks)
        tr, tf, _, res = I.tabu_run(3, 60, -1, V0=V0, stop_on_zero=False)
    assert res == ores and np.array_equal(tr, otr) and np.array_equal(tf, otf)


@pytest.mark.parametrize("m,n,k,blocks,iters", [(300, 50, 3, 1, 25), (300, 50, 3, 3, 25), (400, 120, 2, 1, 30),
                                                 (257, 64, 1, 1, 200)])
def test_large_m_padded_placement_trajectory(L, orc, m, n, k, blocks, iters):
    """m > 255 (segment-loop path) with large CTA slices: budgeted padded placement (DESIGN.md
    §5.4). Random starts give deep-negative rows, empty lattice points and segments of every
    size; the whole trajectory must equal the oracle's."""
    inst = pi.planted_instance(m, n, 7000 + m + n + k)
    V0 = pi.start_vector(n, 11 + k)
    ten = pi.default_tenure(n, k)
    otr, otf, oVo, ores = orc.tabu_run(inst.A, inst.S, k, V0, iters, ten, stop_on_zero=False)
    with L.Instance(inst.A, inst.S) as I:
        L.lns_config(I.ctx, blocks)
        tr, tf, Vo, res = I.tabu_run(k, iters, -1, V0=V0, stop_on_zero=False)
    assert res == ores and np.array_equal(tr, otr) and np.array_equal(tf, otf) and np.array_equal(Vo, oVo)


def _clustered_instance(m, n, npool, noise, seed):
    """Rows drawn from a small pool of +-1 rows (plus noise): many rows share a lattice point, so
    some states exceed the byte window of the packed plan for m > 255 and others do not."""
    rng = np.random.default_rng(seed)
    pool = np.where(rng.random((npool, n)) < 0.5, -1, 1).astype(np.int8)
    A = pool[rng.integers(0, npool, m)].copy()
    A[rng.random((m, n)) < noise] *= -1
    secret = np.where(rng.random(n) < 0.5, -1, 1).astype(np.int8)
    y = A.astype(np.int64) @ secret
    A[y < 0] *= -1
    return A, np.abs(y).astype(np.int32)


@pytest.mark.parametrize("k,iters,m,npool,noise", [(1, 150, 700, 10, 0.1), (2, 60, 550, 8, 0.12),
                                                   (3, 25, 500, 8, 0.12)])
@pytest.mark.parametrize("blocks", [1, 5])
def test_large_m_packed_plan_guard_mixed_trajectory(L, orc, k, iters, m, npool, noise, blocks, monkeypatch):
    """m > 255: each iteration takes the packed byte-window plan when the
    state's counts fit bytes and the segment plan otherwise. On these clustered instances the
    guard (restated in tests/test_packed_model.bytes_fit) switches along the trajectory; the
    whole trajectory must equal the oracle's."""
    from test_packed_model import bytes_fit

    n = 40
    A, S = _clustered_instance(m, n, npool, noise, 100 + k)
    V0 = pi.start_vector(n, 7 + k)
    ten = pi.default_tenure(n, k)
    otr, otf, oVo, ores = orc.tabu_run(A, S, k, V0, iters, ten, stop_on_zero=False)
    V = V0.astype(np.int64).copy()
    fits = []
    for t in range(iters):
        fits.append(bytes_fit(A.astype(np.int64), S, V, k))
        for i in orc.flipsets(n, k, [otr[t]])[0]:
            if i >= 0:
                V[i] = -V[i]
    assert 0 < sum(fits) < iters  # both plans are taken
    monkeypatch.setenv("LNS_FORCE_PKW", "1")  # small slices too (read at create)
    with L.Instance(A, S) as I:
        L.lns_config(I.ctx, blocks)
        tr, tf, Vo, res = I.tabu_run(k, iters, -1, V0=V0, stop_on_zero=False)
        assert res == ores and np.array_equal(tr, otr) and np.array_equal(tf, otf) and np.array_equal(Vo, oVo)
        for Vs in (V0, oVo):
            assert np.array_equal(L.lns_eval_all(I.ctx, k, Vs).astype(np.int64), orc.eval_all(A, S, Vs, k))


@pytest.mark.parametrize("G", [2, 3, 8])
def test_partitioned_search_emulated_on_one_gpu(L, orc, G):
    """The multi-GPU protocol (PAPER.md:448-454 partitioning): G contexts each own a slice of the
    rank space; per iteration every slice's partial key is min-reduced and applied everywhere.
    The trajectory must equal the single-partition one (a u64 MIN of exact keys is associative)."""
    import torch

    inst = pi.config_instance("C4")
    V0 = pi.start_vector(117, 5)
    iters = 40
    otr, otf, oVo, ores = orc.tabu_run(inst.A, inst.S, 3, V0, iters, pi.default_tenure(117, 3), stop_on_zero=False)
    ctxs = [L.lns_create(inst.A, inst.S) for _ in range(G)]
    try:
        keys = torch.empty((G, 1), dtype=torch.int64, device="cuda")
        for g, c in enumerate(ctxs):
            L.lns_set_partition(c, g, G)
            L.lns_step_begin(c, 3, iters, -1, 0, V0, 0)
        for _ in range(iters):
            for g, c in enumerate(ctxs):
                L.lns_step_eval(c, keys[g])
            keys.copy_(keys.min(dim=0, keepdim=True).values.expand(G, 1))
            for g, c in enumerate(ctxs):
                L.lns_step_apply(c, keys[g])
        torch.cuda.synchronize()
        for c in ctxs:
            tr = np.empty(iters, np.int64)
            tf = np.empty(iters, np.int64)
            Vo = np.empty(117, np.int8)
            res = L.lns_step_end(c, Vo, tr, tf)
            assert res == ores and np.array_equal(tr, otr) and np.array_equal(tf, otf)
            assert np.array_equal(Vo, oVo)
    finally:
        for c in ctxs:
            L.lns_destroy(c)


def test_batch_restarts_match_single_runs(L, orc):
    inst = pi.config_instance("C2")
    with L.Instance(inst.A, inst.S) as I:
        R = 4
        Vo = np.empty((R, 73), np.int8)
        batch = L.lns_tabu_run_batch(I.ctx, 2, R, 300, -1, 17, None, L.LNS_STOP_ON_ZERO, Vo)
        for r in range(R):
            V0 = pi.start_vector(73, pi.restart_seed(17, r))
            _, _, oVo, ores = orc.tabu_run(inst.A, inst.S, 2, V0, 300, pi.default_tenure(73, 2))
            assert batch[r] == ores
            assert np.array_equal(Vo[r], oVo)


def test_C5_two_iterations_properties(L, orc):
    """C5 trajectories are beyond the oracle (1.9e14 ops per iteration); check the first two
    iterations by sampled properties: each accepted fitness equals the oracle's from-scratch
    fitness of the resulting vector, and is <= every sampled admissible neighbour's fitness."""
    inst = pi.config_instance("C5")
    seed = pi.config_seed("C5")
    V = pi.start_vector(1024, seed)
    rng = np.random.default_rng(55)
    M = comb(1024, 3)
    with L.Instance(inst.A, inst.S) as I:
        tr, tf, Vo, res = I.tabu_run(3, 2, -1, seed=seed, stop_on_zero=False)
    assert res["iters_done"] == 2
    for t in range(2):
        sample = np.unique(rng.integers(0, M, 2000))
        sample = sample[~np.isin(sample, tr[:t])]
        fs = orc.eval_ranks(inst.A, inst.S, V, 3, sample)
        assert tf[t] <= fs.min()
        (f3,) = orc.flipsets(1024, 3, [tr[t]])
        V = V.copy()
        V[f3] *= -1
        assert orc.fitness(inst.A, inst.S, V, packed=True) == tf[t]
    assert np.array_equal(V, Vo)


def test_python_partitioned_driver_with_nccl_world1(L, orc):
    """parallel.partitioned_tabu_run + LnsStepper over a real NCCL process group (world 1): the
    Python-driven protocol gives the oracle trajectory."""
    import os

    import torch
    import torch.distributed as dist

    from paper_conf_ipps_luongmt10_b200 import parallel as par

    os.environ.setdefault("MASTER_ADDR", "127.0.0.1")
    os.environ.setdefault("MASTER_PORT", "29533")
    dist.init_process_group("nccl", rank=0, world_size=1, device_id=torch.device("cuda", 0))
    try:
        inst = pi.config_instance("C3")
        V0 = pi.start_vector(81, 3)
        ctx = L.lns_create(inst.A, inst.S)
        try:
            st = par.LnsStepper(ctx, 81, 3, 30, -1, 0, V0, stop_on_zero=False, rank=0, world=1)
            tr, tf, Vo, res = par.partitioned_tabu_run(st, 30)
        finally:
            L.lns_destroy(ctx)
        otr, otf, oVo, ores = orc.tabu_run(inst.A, inst.S, 3, V0, 30, pi.default_tenure(81, 3), stop_on_zero=False)
        assert res == ores and np.array_equal(tr, otr) and np.array_equal(tf, otf) and np.array_equal(Vo, oVo)
    finally:
        dist.destroy_process_group()


@pytest.mark.parametrize("cfg,R,iters,stop", [("C1", 300, 200, True), ("C2", 20, 150, False), ("C3", 6, 40, False),
                                              ("C4", 3, 25, False)])
def test_batched_restarts_grouped_kernel(L, orc, cfg, R, iters, stop):
    """lns_tabu_run_batch splits the grid into groups, each running whole searches (C1 with 300
    restarts: more restarts than SMs, so groups run several in turn). Every restart must equal the
    oracle's search from splitmix64(seed + r) (reading R12)."""
    c = pi.CONFIGS[cfg]
    inst = pi.config_instance(cfg)
    seed = 1234
    ten = pi.default_tenure(inst.n, c["k"])
    with L.Instance(inst.A, inst.S) as I:
        Vo = np.empty((R, inst.n), np.int8)
        batch = L.lns_tabu_run_batch(I.ctx, c["k"], R, iters, -1, seed, None,
                                     L.LNS_STOP_ON_ZERO if stop else 0, Vo)
    check = range(R) if R <= 20 else list(range(0, R, 7)) + [R - 1]
    for r in check:
        V0 = pi.start_vector(inst.n, pi.restart_seed(seed, r))
        _, _, oVo, ores = orc.tabu_run(inst.A, inst.S, c["k"], V0, iters, ten, stop_on_zero=stop)
        assert batch[r] == ores, r
        assert np.array_equal(Vo[r], oVo), r


@pytest.mark.parametrize("cfg,R,iters", [("C4", 50, 12), ("C3", 50, 30), ("C2", 149, 40)])
def test_batched_two_phase_schedule(L, orc, cfg, R, iters):
    """The bench's job shape: the makespan model splits R searches into two phases with different
    CTAs per search (C4/C3, 50 runs: one search on every SM, then 49 searches on 3 CTAs each;
    C2, 149 runs: more searches than SMs). Sampled runs of both phases must equal the oracle."""
    c = pi.CONFIGS[cfg]
    inst = pi.config_instance(cfg)
    seed = 99
    ten = pi.default_tenure(inst.n, c["k"])
    with L.Instance(inst.A, inst.S) as I:
        Vo = np.empty((R, inst.n), np.int8)
        batch = L.lns_tabu_run_batch(I.ctx, c["k"], R, iters, -1, seed, None, 0, Vo)
    for r in (0, 1, R // 2, R - 2, R - 1):
        V0 = pi.start_vector(inst.n, pi.restart_seed(seed, r))
        _, _, oVo, ores = orc.tabu_run(inst.A, inst.S, c["k"], V0, iters, ten, stop_on_zero=False)
        assert batch[r] == ores, r
        assert np.array_equal(Vo[r], oVo), r


def test_bench_job_full_size_sampled_runs(L, orc):
    """The bench's timed job exactly as bench.py launches it (C4, 50 searches x 400 iterations,
    tenure floor(M/6), start vectors of bench step 3 from device memory, the two-phase schedule):
    sampled runs of both phases -- final result and final vector -- equal the oracle run for the
    full 400 iterations."""
    import sys

    import torch

    sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
    import bench

    inst = pi.config_instance(bench.CFG)
    ten = pi.default_tenure(inst.n, 3)
    step = 3  # the first timed step of a default run (warm-up 3)
    V0 = bench.start_vectors(inst.n, step, range(bench.RUNS))
    with L.Instance(inst.A, inst.S) as I:
        Vo = torch.empty((bench.RUNS, inst.n), dtype=torch.int8, device="cuda")
        res = L.lns_tabu_run_batch(I.ctx, 3, bench.RUNS, bench.ITERS, ten, 0, torch.from_numpy(V0).cuda(), 0, Vo)
        Vo = Vo.cpu().numpy()
    for r in (0, 1, 25, bench.RUNS - 1):
        _, _, oVo, ores = orc.tabu_run(inst.A, inst.S, 3, V0[r], bench.ITERS, ten, stop_on_zero=False)
        assert res[r] == ores, r
        assert np.array_equal(Vo[r], oVo), r


def test_batched_restarts_given_start_vectors(L, orc):
    inst = pi.planted_instance(45, 37, 31)
    rng = np.random.default_rng(3)
    V0 = np.where(rng.random((9, 37)) < 0.5, -1, 1).astype(np.int8)
    with L.Instance(inst.A, inst.S) as I:
        Vo = np.empty((9, 37), np.int8)
        batch = L.lns_tabu_run_batch(I.ctx, 3, 9, 60, 11, 0, V0, 0, Vo)
    for r in range(9):
        _, _, oVo, ores = orc.tabu_run(inst.A, inst.S, 3, V0[r], 60, 11, stop_on_zero=False)
        assert batch[r] == ores and np.array_equal(Vo[r], oVo)


@pytest.mark.parametrize("k,L_ten,iters", [(1, 5, 200), (2, 100, 150), (3, 2000, 80)])
def test_aspiration_variant_bit_exact(L, orc, k, L_ten, iters):
    """LNS_ASPIRATION (variant R4'): persistent, stepped and batched paths against the oracle."""
    inst = pi.planted_instance(41, 35, 800 + k)
    V0 = pi.start_vector(35, 60 + k)
    otr, otf, oVo, ores = orc.tabu_run(inst.A, inst.S, k, V0, iters, L_ten, stop_on_zero=False, aspiration=True)
    with L.Instance(inst.A, inst.S) as I:
        for flags in (L.LNS_ASPIRATION, L.LNS_ASPIRATION | L.LNS_FORCE_STEPPED):
            tr, tf, Vo, res = I.tabu_run(k, iters, L_ten, V0=V0, stop_on_zero=False, flags=flags)
            assert res == ores and np.array_equal(tr, otr) and np.array_equal(tf, otf)
        Vb = np.empty((1, 35), np.int8)
        batch = L.lns_tabu_run_batch(I.ctx, k, 1, iters, L_ten, 0, V0[None, :], L.LNS_ASPIRATION, Vb)
        assert batch[0] == ores and np.array_equal(Vb[0], oVo)


@pytest.mark.parametrize("k,L_ten,iters,blocks", [(1, 4, 200, 1), (1, 30, 200, 3), (2, 1, 120, 2), (2, 50, 150, 5),
                                                  (3, 7, 80, 4), (3, -1, 60, 148)])
@pytest.mark.parametrize("aspiration", [False, True])
def test_solution_list_variant_bit_exact(L, orc, k, L_ten, iters, blocks, aspiration):
    """LNS_TABU_SOLUTIONS (variant R3', PAPER.md:243-244 read literally): the tabu list holds the
    L most recently visited solutions. Persistent kernel on 1..148 CTAs (the group barrier that
    publishes the scanned ranks) and batched restarts, against the oracle's hash-set variant.
    Short tenures wrap the visited ring many times."""
    inst = pi.planted_instance(41, 35, 900 + k)
    V0 = pi.start_vector(35, 80 + k)
    ten = pi.default_tenure(35, k) if L_ten < 0 else L_ten
    otr, otf, oVo, ores = orc.tabu_run(inst.A, inst.S, k, V0, iters, ten, stop_on_zero=False,
                                       aspiration=aspiration, tabu_solutions=True)
    flags = L.LNS_TABU_SOLUTIONS | (L.LNS_ASPIRATION if aspiration else 0)
    with L.Instance(inst.A, inst.S) as I:
        L.lns_config(I.ctx, blocks)
        tr, tf, Vo, res = I.tabu_run(k, iters, L_ten, V0=V0, stop_on_zero=False, flags=flags)
        assert res == ores and np.array_equal(tr, otr) and np.array_equal(tf, otf) and np.array_equal(Vo, oVo)
        L.lns_config(I.ctx, 0)
        Vb = np.empty((3, 35), np.int8)
        V0s = np.stack([V0, pi.start_vector(35, 1), pi.start_vector(35, 2)])
        batch = L.lns_tabu_run_batch(I.ctx, k, 3, iters, L_ten, 0, V0s, flags, Vb)
    assert batch[0] == ores and np.array_equal(Vb[0], oVo)
    for r in (1, 2):
        _, _, oV, orr = orc.tabu_run(inst.A, inst.S, k, V0s[r], iters, ten, stop_on_zero=False,
                                     aspiration=aspiration, tabu_solutions=True)
        assert batch[r] == orr and np.array_equal(Vb[r], oV)


def test_solution_list_variant_C3_and_errors(L, orc):
    """C3 shape (85,320 neighbours, 148 CTAs, the flip-set cache) with the solution list of the
    paper's size L = C(n,3)/6, and the argument errors: tenure 0, the stepped path."""
    inst = pi.config_instance("C3")
    V0 = pi.start_vector(81, 3)
    ten = pi.default_tenure(81, 3)
    otr, otf, oVo, ores = orc.tabu_run(inst.A, inst.S, 3, V0, 40, ten, stop_on_zero=False, tabu_solutions=True)
    with L.Instance(inst.A, inst.S) as I:
        tr, tf, Vo, res = I.tabu_run(3, 40, -1, V0=V0, stop_on_zero=False, flags=L.LNS_TABU_SOLUTIONS)
        assert res == ores and np.array_equal(tr, otr) and np.array_equal(tf, otf) and np.array_equal(Vo, oVo)
        for ten_bad, fl in ((0, L.LNS_TABU_SOLUTIONS), (5, L.LNS_TABU_SOLUTIONS | L.LNS_FORCE_STEPPED)):
            with pytest.raises(L.LnsError) as ei:
                I.tabu_run(3, 5, ten_bad, V0=V0, stop_on_zero=False, flags=fl)
            assert ei.value.status == L.LNS_EINVAL
        with pytest.raises(L.LnsError) as ei:
            L.lns_step_begin(I.ctx, 3, 5, 5, 0, V0, L.LNS_TABU_SOLUTIONS)
        assert ei.value.status == L.LNS_EINVAL


@pytest.mark.parametrize("k", [1, 2])
def test_large_instance_global_X_fallback(L, orc, k):
    """1201 x 1217 (the Fig. 8 ladder): the sorted sign bits X no longer fit in
    shared memory, so each CTA keeps them in global memory. All fitnesses (k = 1) or a sample
    (k = 2) and a short k = 1 trajectory against the oracle."""
    inst = pi.planted_instance(1201, 1217, 4321)
    V = pi.start_vector(1217, 77)
    M = comb(1217, k)
    with L.Instance(inst.A, inst.S) as I:
        got = L.lns_eval_all(I.ctx, k, V).astype(np.int64)
        if k == 1:
            assert np.array_equal(got, orc.eval_all(inst.A, inst.S, V, 1))
            tr, tf, Vo, res = I.tabu_run(1, 40, -1, V0=V, stop_on_zero=False)
            otr, otf, oVo, ores = orc.tabu_run(inst.A, inst.S, 1, V, 40, pi.default_tenure(1217, 1), stop_on_zero=False)
            assert res == ores and np.array_equal(tr, otr) and np.array_equal(Vo, oVo)
        else:
            ranks = np.unique(np.random.default_rng(2).integers(0, M, 4000))
            assert np.array_equal(got[ranks], orc.eval_ranks(inst.A, inst.S, V, 2, ranks))


@pytest.mark.parametrize("m,n,k", [(m, n, k) for (m, n, k) in SHAPES if comb(n, k) >= 4096])
def test_eval_all_large_slices(L, orc, m, n, k):
    """One CTA for the whole neighbourhood: slices of >= 4 block passes take the batched-search
    evaluation path (two neighbours per thread over contiguous rank runs, lexicographic successor)
    and, for m <= 255, the padded row placement -- every fitness vs the oracle."""
    inst = pi.planted_instance(m, n, 7000 + m * 31 + n)
    rng = np.random.default_rng(m * n + k + 1)
    ctx = L.lns_create(inst.A, inst.S)
    try:
        L.lns_config(ctx, 1)
        for V in _states(inst, rng, count=2):
            got = L.lns_eval_all(ctx, k, V)
            want = orc.eval_all(inst.A, inst.S, V, k)
            assert np.array_equal(got.astype(np.int64), want)
    finally:
        L.lns_destroy(ctx)


@pytest.mark.parametrize("m,n,k", [(300, 50, 3), (260, 40, 2), (520, 64, 1), (1024, 200, 2), (700, 90, 3)])
@pytest.mark.parametrize("plan", ["LNS_FORCE_PKW", "LNS_NO_PKW"])
def test_eval_all_large_m_both_plans(L, orc, m, n, k, plan, monkeypatch):
    """m > 255: every fitness with the packed plan tried on every slice
    (LNS_FORCE_PKW; states whose counts fit bytes take it) and with the segment plan only
    (LNS_NO_PKW), against the oracle."""
    monkeypatch.setenv(plan, "1")
    inst = pi.planted_instance(m, n, 8100 + m + n + k)
    rng = np.random.default_rng(m + n + k)
    ctx = L.lns_create(inst.A, inst.S)
    try:
        for V in _states(inst, rng, count=1):
            got = L.lns_eval_all(ctx, k, V)
            assert np.array_equal(got.astype(np.int64), orc.eval_all(inst.A, inst.S, V, k))
    finally:
        L.lns_destroy(ctx)


# ------------------------------------------------------------------ device-initiated exchange (f3)
def _peer_pair(L, inst, nb):
    ctxs = [L.lns_create(inst.A, inst.S) for _ in range(2)]
    for c in ctxs:
        L.lns_config(c, nb)
    bufs = [L.lns_exchange_buffer(c) for c in ctxs]
    return ctxs, bufs


@pytest.mark.parametrize("cfg,iters,sols", [("C4", 120, False), ("C3", 300, False), ("C2", 400, False),
                                           ("C3", 150, True)])
def test_peer_exchange_two_partitions_one_gpu(L, orc, cfg, iters, sols):
    """two partitions, each a persistent kernel of 32 CTAs on its own stream,
    exchange the per-iteration MIN through each other's exchange buffers (red.min.sys /
    red.release.sys / ld.acquire.sys) with no host step. Both must reproduce the single-context
    trajectory bit for bit (same device here, so plain launches: the driver serialises cooperative
    ones; across GPUs the buffers are NVLink peer memory and each GPU runs one cooperative kernel)."""
    import threading

    import torch

    c = pi.CONFIGS[cfg]
    inst = pi.config_instance(cfg)
    k, n = c["k"], inst.n
    V0 = pi.start_vector(n, pi.config_seed(cfg))
    fl = L.LNS_TABU_SOLUTIONS if sols else 0  # the solution list (R3') is scanned per partition
    # the reference is the ORACLE's trajectory, not a single-context GPU run
    tr0, tf0, v0, r0 = orc.tabu_run(inst.A, inst.S, k, V0, iters, pi.default_tenure(n, k), stop_on_zero=False,
                                    tabu_solutions=sols)
    ctxs, bufs = _peer_pair(L, inst, 32)
    try:
        # a plain run first: every buffer the run needs is allocated now (cudaMalloc synchronises
        # the device, which would serialise the two partitions' kernels in one process)
        for cx in ctxs:
            L.lns_tabu_run(cx, k, iters, -1, 0, V0, fl)
        for p, cx in enumerate(ctxs):
            L.lns_attach_peers(cx, p, 2, bufs, 20000)
        for cx in ctxs:
            L.lns_exchange_reset(cx)
        outs = [dict(tr=np.zeros(iters, np.int64), tf=np.zeros(iters, np.int64), v=np.zeros(n, np.int8))
                for _ in ctxs]
        errs = [None, None]
        streams = [torch.cuda.Stream() for _ in ctxs]

        def run(p):
            try:
                o = outs[p]
                o["res"] = L.lns_tabu_run(ctxs[p], k, iters, -1, 0, V0, L.LNS_PLAIN_LAUNCH | fl, o["v"], o["tr"], o["tf"],
                                          streams[p])
            except Exception as e:  # noqa: BLE001 - reported below
                errs[p] = e

        th = [threading.Thread(target=run, args=(p,)) for p in range(2)]
        for t in th:
            t.start()
        for t in th:
            t.join()
        assert errs == [None, None], errs
        for o in outs:
            assert np.array_equal(o["tr"], tr0) and np.array_equal(o["tf"], tf0)
            assert np.array_equal(o["v"], v0) and o["res"] == r0
    finally:
        for cx in ctxs:
            L.lns_destroy(cx)


def test_peer_exchange_missing_partition_times_out(L):
    """A partition that never arrives ends the run with LNS_EPEER after the timeout (no hang)."""
    inst = pi.config_instance("C3")
    ctxs, bufs = _peer_pair(L, inst, 16)
    try:
        L.lns_attach_peers(ctxs[0], 0, 2, bufs, 300)
        L.lns_exchange_reset(ctxs[0])
        with pytest.raises(L.LnsError) as ei:
            L.lns_tabu_run(ctxs[0], 3, 50, -1, 0, pi.start_vector(inst.n, 4), 0)
        assert ei.value.status == L.LNS_EPEER
        L.lns_attach_peers(ctxs[0], 0, 1, None)  # detached: a plain run works again
        res = L.lns_tabu_run(ctxs[0], 3, 5, -1, 0, pi.start_vector(inst.n, 4), 0)
        assert res["iters_done"] == 5
    finally:
        for cx in ctxs:
            L.lns_destroy(cx)


def test_pool_recycles_context_buffers(L, orc):
    """create -> batch -> destroy cycles reuse the library's cached device blocks (include/lns.h,
    device-memory cache): the second cycle allocates nothing new, every block is returned at
    destroy, and recycled (not re-zeroed) buffers give the same oracle-exact results."""
    inst = pi.config_instance("C3")
    seed, R, iters = 77, 4, 30
    ten = pi.default_tenure(inst.n, 3)
    outs, footprint = [], []
    for _ in range(3):
        ctx = L.lns_create(inst.A, inst.S, 0)
        Vo = np.empty((R, inst.n), np.int8)
        outs.append((L.lns_tabu_run_batch(ctx, 3, R, iters, -1, seed, None, 0, Vo), Vo.copy()))
        cached, live = L.lns_pool_stats()
        assert live > 0
        L.lns_destroy(ctx)
        cached2, live2 = L.lns_pool_stats()
        assert cached2 == cached + live and live2 == 0
        footprint.append(cached2)
    assert footprint[1] == footprint[0] == footprint[2]
    for res, Vo in outs[1:]:
        assert res == outs[0][0] and np.array_equal(Vo, outs[0][1])
    V0 = pi.start_vector(inst.n, pi.restart_seed(seed, 1))
    _, _, oVo, ores = orc.tabu_run(inst.A, inst.S, 3, V0, iters, ten, stop_on_zero=False)
    assert outs[2][0][1] == ores and np.array_equal(outs[2][1][1], oVo)
    L.lns_pool_trim()
    assert L.lns_pool_stats() == (0, 0)


@pytest.mark.parametrize("tool", ["memcheck", "racecheck", "synccheck"])
def test_compute_sanitizer_clean(L, tool):
    """every kernel family (persistent search with one and several CTAs,
    batched restarts, stepped search, eval_all, the m > 255 path, the UBQP kernels) runs clean under
    compute-sanitizer on small instances.

    Opt-in (LNS_SANITIZE=1): the GPU pool this round runs on has closed compute-sanitizer (runs
    under it left GPUs needing a reset), so the default suite does not start it. Round 1 ran all
    three tools clean; the bounds-checked parity tests below stand in for it."""
    import os
    import shutil
    import subprocess
    import sys

    if os.environ.get("LNS_SANITIZE") != "1":
        pytest.skip("compute-sanitizer is opt-in (LNS_SANITIZE=1): closed on this GPU pool")
    exe = shutil.which("compute-sanitizer") or "/usr/local/cuda/bin/compute-sanitizer"
    if not os.path.exists(exe):
        pytest.skip("compute-sanitizer not found")
    root = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
    cmd = [exe, "--tool", tool, "--error-exitcode", "9", sys.executable, os.path.join(root, "scripts", "sanitize_probe.py")]
    out = subprocess.run(cmd, capture_output=True, text=True, timeout=900, cwd=root)
    tail = (out.stdout + out.stderr)[-3000:]
    assert out.returncode == 0, tail
    assert "sanitize probe done" in out.stdout, tail
    log = out.stdout + out.stderr
    assert "ERROR SUMMARY: 0 errors" in log or "SUMMARY: 0 hazards displayed (0 errors" in log, tail


# ------------------------------------------------------------------ k > 3
@pytest.mark.parametrize("k", [4, 5, 6, 7])
def test_unrank_k_above_3_exhaustive(L, orc, k):
    for n in (k, k + 1, 13, 30 if k < 7 else 24):
        M = comb(n, k)
        r = np.arange(M, dtype=np.int64)
        assert np.array_equal(L.lns_unrank(n, k, r), orc.flipsets(n, k, r))


@pytest.mark.parametrize("n,k", [(500, 4), (200, 5), (120, 6), (80, 7)])
def test_unrank_k_above_3_sampled_large(L, n, k):
    """Large n: sampled ranks (both ends included) map to strictly increasing index tuples whose
    lexicographic rank, restated with math.comb, is the rank itself."""
    M = comb(n, k)
    rng = np.random.default_rng(n + k)
    r = np.unique(np.concatenate([[0, 1, M - 2, M - 1], rng.integers(0, M, 3000)])).astype(np.int64)
    F = L.lns_unrank(n, k, r)
    assert np.all(np.diff(F, axis=1) > 0) and F.min() >= 0 and F.max() < n
    for q in range(0, len(r), 97):
        lex = M - 1 - sum(comb(n - 1 - int(F[q, j]), k - j) for j in range(k))
        assert lex == r[q]


@pytest.mark.parametrize("m,n,k", [(41, 35, 4), (70, 40, 4), (33, 23, 5), (100, 20, 6), (255, 18, 7)])
def test_eval_all_k_above_3_matches_oracle(L, orc, m, n, k):
    """Every neighbour's fitness for k = 4..7 (random, near-secret, all-negative and secret
    states: deep rows, rows above the top cut, empty lattice points, m up to 255)."""
    inst = pi.planted_instance(m, n, 4000 + m + k)
    rng = np.random.default_rng(m * n + k)
    with L.Instance(inst.A, inst.S) as I:
        for V in _states(inst, rng, count=1):
            got = L.lns_eval_all(I.ctx, k, V).astype(np.int64)
            assert np.array_equal(got, orc.eval_all(inst.A, inst.S, V, k))


@pytest.mark.parametrize("k,ten,iters,blocks", [(4, -1, 30, 0), (4, 5, 40, 3), (5, 0, 20, 1), (6, 50, 12, 0)])
@pytest.mark.parametrize("aspiration", [False, True])
def test_trajectory_k_above_3_bit_exact(L, orc, k, ten, iters, blocks, aspiration):
    inst = pi.planted_instance(45, 29, 5000 + k)
    V0 = pi.start_vector(29, 30 + k)
    t_or = pi.default_tenure(29, k) if ten < 0 else ten
    otr, otf, oVo, ores = orc.tabu_run(inst.A, inst.S, k, V0, iters, t_or, stop_on_zero=False, aspiration=aspiration)
    with L.Instance(inst.A, inst.S) as I:
        L.lns_config(I.ctx, blocks)
        tr, tf, Vo, res = I.tabu_run(k, iters, ten, V0=V0, stop_on_zero=False,
                                     flags=L.LNS_ASPIRATION if aspiration else 0)
    assert res == ores and np.array_equal(tr, otr) and np.array_equal(tf, otf) and np.array_equal(Vo, oVo)


def test_k_above_3_limits(L):
    inst = pi.planted_instance(300, 20, 9)
    small = pi.planted_instance(20, 12, 9)
    with L.Instance(inst.A, inst.S) as I:
        with pytest.raises(L.LnsError) as ei:
            I.tabu_run(4, 3, -1, seed=1)
        assert ei.value.status == L.LNS_ERANGE  # m > 255
    with L.Instance(small.A, small.S) as I:
        for call in (lambda: L.lns_tabu_run_batch(I.ctx, 4, 2, 3, 2, 0, None, L.LNS_TABU_SOLUTIONS),
                     lambda: I.tabu_run(8, 3, -1, seed=1),
                     lambda: I.tabu_run(4, 3, -1, seed=1, flags=L.LNS_FORCE_STEPPED),
                     lambda: I.tabu_run(4, 3, 2, seed=1, flags=L.LNS_TABU_SOLUTIONS)):
            with pytest.raises(L.LnsError) as ei:
                call()
            assert ei.value.status == L.LNS_EINVAL
        res = I.tabu_run(4, 5, -1, seed=1, stop_on_zero=False)[3]
        assert res["iters_done"] == 5


@pytest.mark.parametrize("k,R,iters,blocks,aspiration", [(4, 5, 25, 0, False), (4, 9, 15, 2, True), (5, 3, 10, 0, False),
                                                         (4, 200, 6, 0, False)])
def test_batch_k_above_3_matches_single_runs(L, orc, k, R, iters, blocks, aspiration):
    """lns_tabu_run_batch for k >= 4: groups of CTAs run whole restarts (in-kernel restart init,
    per-group exchange and until[]); R > SMs takes several restarts per group."""
    inst = pi.planted_instance(37, 26, 5100 + k)
    rng = np.random.default_rng(R + k)
    V0 = np.where(rng.random((R, 26)) < 0.5, -1, 1).astype(np.int8)
    fl = L.LNS_ASPIRATION if aspiration else 0
    with L.Instance(inst.A, inst.S) as I:
        L.lns_config(I.ctx, blocks)
        Vo = np.empty((R, 26), np.int8)
        batch = L.lns_tabu_run_batch(I.ctx, k, R, iters, -1, 0, V0, fl, Vo)
    for r in sorted(set(range(0, R, max(1, R // 8))) | {R - 1}):
        _, _, oVo, ores = orc.tabu_run(inst.A, inst.S, k, V0[r], iters, pi.default_tenure(26, k),
                                       stop_on_zero=False, aspiration=aspiration)
        assert batch[r] == ores and np.array_equal(Vo[r], oVo), r


def _nccl_world1_comm():
    """A one-rank NCCL communicator created through the libnccl torch ships (ctypes:
    ncclGetUniqueId + ncclCommInitRank), for the production lns_attach_comm path."""
    import ctypes
    import glob
    import os

    import nvidia

    libs = glob.glob(os.path.join(list(nvidia.__path__)[0], "nccl", "lib", "libnccl.so*"))
    if not libs:
        pytest.skip("libnccl not found")
    class UniqueId(ctypes.Structure):  # ncclUniqueId: 128 bytes, passed by value
        _fields_ = [("internal", ctypes.c_char * 128)]

    nccl = ctypes.CDLL(libs[0], mode=ctypes.RTLD_GLOBAL)
    uid = UniqueId()
    assert nccl.ncclGetUniqueId(ctypes.byref(uid)) == 0
    comm = ctypes.c_void_p()
    nccl.ncclCommInitRank.argtypes = [ctypes.POINTER(ctypes.c_void_p), ctypes.c_int, UniqueId, ctypes.c_int]
    assert nccl.ncclCommInitRank(ctypes.byref(comm), 1, uid, 0) == 0
    return nccl, comm


@pytest.mark.parametrize("cfg,iters", [("C2", 300), ("C3", 140)])
def test_nccl_attached_stepped_loop_with_graphs(L, orc, cfg, iters, monkeypatch):
    """lns_attach_comm with a real NCCL communicator (world 1): the stepped loop of lns_tabu_run
    (eval launch, ncclAllReduce u64 MIN, apply launch per iteration) captured into CUDA graphs of
    64 iterations and replayed, plus direct iterations; and the same with LNS_NO_GRAPH=1. Both
    give the oracle trajectory."""
    import torch

    torch.cuda.init()
    nccl, comm = _nccl_world1_comm()
    c = pi.CONFIGS[cfg]
    inst = pi.config_instance(cfg)
    V0 = pi.start_vector(inst.n, 5)
    otr, otf, oVo, ores = orc.tabu_run(inst.A, inst.S, c["k"], V0, iters, pi.default_tenure(inst.n, c["k"]),
                                       stop_on_zero=False)
    try:
        for nog in ("0", "1"):
            monkeypatch.setenv("LNS_NO_GRAPH", nog)
            with L.Instance(inst.A, inst.S) as I:
                L.lns_attach_comm(I.ctx, comm.value, 0, 1)
                tr, tf, Vo, res = I.tabu_run(c["k"], iters, -1, V0=V0, stop_on_zero=False)
                L.lns_attach_comm(I.ctx, None, 0, 1)
            assert res == ores and np.array_equal(tr, otr) and np.array_equal(tf, otf) and np.array_equal(Vo, oVo)
    finally:
        nccl.ncclCommDestroy(comm)


@pytest.mark.parametrize("m,n,k", [(41, 30, 4), (60, 22, 5)])
def test_eval_neighborhood_k_above_3_best_with_tabu(L, orc, m, n, k):
    """lns_eval_neighborhood for k >= 4: best admissible (f, rank) with 0 / 50 % / all-but-one tabu,
    and ENOADMISSIBLE when every rank is tabu."""
    inst = pi.planted_instance(m, n, 5300 + n + k)
    rng = np.random.default_rng(n + k)
    M = comb(n, k)
    with L.Instance(inst.A, inst.S) as I:
        for V in _states(inst, rng, count=1):
            Y = (inst.A.astype(np.int32) @ V.astype(np.int32)).astype(np.int32)
            for frac in (0.0, 0.5, 1.0):
                tabu = rng.random(M) < frac
                if frac == 1.0:
                    tabu[rng.integers(M)] = False
                bits = np.packbits(tabu, bitorder="little")
                bits = np.concatenate([bits, np.zeros((-len(bits)) % 4, np.uint8)]).view(np.uint32)
                assert L.lns_eval_neighborhood(I.ctx, k, V, Y, bits) == orc.eval_best(inst.A, inst.S, V, k, tabu)
        allbits = np.full((M + 31) // 32, 0xFFFFFFFF, np.uint32)
        with pytest.raises(L.LnsError) as ei:
            L.lns_eval_neighborhood(I.ctx, k, V, Y, allbits)
        assert ei.value.status == L.LNS_ENOADMISSIBLE


def test_c_example_runs_on_the_gpu(L, tmp_path):
    """examples/tabu_c.c -- the C ABI from plain C, host buffers only: eval, tabu run, batch, and the
    UBQP calls (eval_all, tabu_run: the first move is the best neighbour of x0)."""
    import subprocess

    from test_abi import _build_c_example

    exe = _build_c_example(tmp_path)
    for args in (["101", "117", "3", "200"], ["73", "73", "2", "300"], ["41", "30", "4", "20"]):
        out = subprocess.run([exe, *args], capture_output=True, text=True, timeout=300)
        assert out.returncode == 0 and out.stdout.strip().endswith("ok"), out.stdout + out.stderr


@pytest.mark.parametrize("cfg,iters", [("C3", 90), ("C4", 40)])
def test_nccl_bootstrap_without_torch_comm(L, orc, cfg, iters):
    """lns_get_unique_id + lns_comm_init_rank (include/lns.h, NCCL bootstrap for plain-C callers):
    a communicator created and owned by the context (world 1 on this one-GPU box) drives the
    partitioned loop of lns_tabu_run (eval, ncclAllReduce u64 MIN, apply) and
    lns_tabu_run_batch; both give the oracle's trajectories. Detaching destroys it."""
    c = pi.CONFIGS[cfg]
    inst = pi.config_instance(cfg)
    k, ten = c["k"], pi.default_tenure(inst.n, c["k"])
    V0 = pi.start_vector(inst.n, 11)
    otr, otf, oVo, ores = orc.tabu_run(inst.A, inst.S, k, V0, iters, ten, stop_on_zero=False)
    uid = L.lns_get_unique_id()
    assert len(uid) == L.LNS_UNIQUE_ID_BYTES and any(uid)
    with L.Instance(inst.A, inst.S) as I:
        L.lns_comm_init_rank(I.ctx, uid, 0, 1)
        tr, tf, Vo, res = I.tabu_run(k, iters, -1, V0=V0, stop_on_zero=False)
        assert res == ores and np.array_equal(tr, otr) and np.array_equal(tf, otf) and np.array_equal(Vo, oVo)
        R, seed = 3, 21
        Vb = np.zeros((R, inst.n), np.int8)
        rb = L.lns_tabu_run_batch(I.ctx, k, R, iters // 3, -1, seed, None, 0, Vb)
        for r in range(R):
            v0 = pi.start_vector(inst.n, pi.restart_seed(seed, r))
            _, _, ov, ors = orc.tabu_run(inst.A, inst.S, k, v0, iters // 3, ten, stop_on_zero=False)
            assert rb[r] == ors and np.array_equal(Vb[r], ov)
        L.lns_attach_comm(I.ctx, None, 0, 1)  # destroys the owned communicator
        tr2, _, _, res2 = I.tabu_run(k, 5, -1, V0=V0, stop_on_zero=False)
        assert np.array_equal(tr2, otr[:5])
    with pytest.raises(L.LnsError) as ei:
        L.lns_comm_init_rank(0, uid, 0, 1)
    assert ei.value.status == L.LNS_EINVAL
