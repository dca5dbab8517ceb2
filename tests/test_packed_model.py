"""CPU model of the packed evaluation path, checked against the oracle.

The sm_100a kernel evaluates a neighbour from a per-iteration *plan* (build_plan_pk): rows sorted
by lattice point, two parity walks, padded placement, 16-byte records, a 32-bit byte window per
walk, absorbed empty points, a deep-row constant and a trailing SAD. This file restates that
arithmetic in plain Python -- record by record, with the same byte-level instructions (prmt,
idp.2a, vabsdiff4, funnel shift) -- and checks the fitness it produces against the oracle's
from-scratch fitness for random instances, states and flip sets, so the design
is pinned on a host without a GPU. It is a model for the tests only: the product path never runs
it, and the GPU parity tests (test_gpu_parity.py) check the kernels themselves.
"""
import numpy as np
import pytest

import oracle
import ppp_inputs as pi

M32 = 0xFFFFFFFF


def popc(x):
    return bin(x & M32).count("1")


def prmt(a, b, sel):
    src = [(a >> (8 * i)) & 255 for i in range(4)] + [(b >> (8 * i)) & 255 for i in range(4)]
    return sum(src[(sel >> (4 * i)) & 7] << (8 * i) for i in range(4))


def vabsdiff4_add(a, b, c):
    return (c + sum(abs(((a >> (8 * i)) & 255) - ((b >> (8 * i)) & 255)) for i in range(4))) & M32


def dp2a_lo(a, b, c):
    return (c + (a & 0xFFFF) * (b & 255) + ((a >> 16) & 0xFFFF) * ((b >> 8) & 255)) & M32


def build_plan(A, S, V, K, pad):
    """build_plan_pk: placement deep | walk 0 | walk 1 | top, records, walk constants, X."""
    m, n = A.shape
    Y = A @ V
    H = np.bincount(S, minlength=n + 1)
    maxS = max(b for b in range(n + 1) if H[b] > 0)
    vmin = int(Y.min())
    U = (int(Y.max()) - vmin) // 2 + 1
    cnt = [int(((Y - vmin) // 2 == u).sum()) for u in range(U)]
    uneg = min(max((-2 * K - vmin + 1) >> 1, 0), U)
    utop = min(max(((maxS + 2 * K - vmin) >> 1) + 1, uneg), U)
    n0, n1 = (utop - uneg + 1) >> 1, (utop - uneg) >> 1
    order = list(range(uneg)) + [uneg + 2 * i for i in range(n0)] + [uneg + 1 + 2 * i for i in range(n1)] \
        + list(range(utop, U))
    pos = runp = prev = 0
    seg, pofs = {}, {}
    rneg, rtop = sum(cnt[:uneg]), sum(cnt[:utop])
    pkb1 = None
    for qi, v in enumerate(order):
        L = cnt[v]
        walk = uneg <= qi < utop
        if qi == uneg + n0:
            pkb1, prev = runp, 0
        if walk and pad and L > 0 and pos % 32 and pos % 32 + L > 32:
            pos = (pos + 31) // 32 * 32
        nonneg = vmin + 2 * (v - K) >= 0
        if pad:  # sequential rule of the padded placement
            absorbed = walk and L == 0 and nonneg and prev == 2
        else:    # warp-scan rule of the unpadded placement
            absorbed = walk and L == 0 and nonneg and v - 2 >= uneg and vmin + 2 * (v - 2 - K) >= 0 and cnt[v - 2] > 0
        seg[v], pofs[v] = pos, (-1 if absorbed else runp)
        if walk:
            runp += ((pos + L - 1) // 32 - pos // 32 + 1) if L > 0 else (0 if absorbed else 1)
            prev = 1 if absorbed else (2 if nonneg else 1)
        pos += L
    if pkb1 is None:
        pkb1 = runp
    Wp = (pos + 31) // 32
    rowAt = [-1] * (32 * Wp)
    cur = dict(seg)
    for j in range(m):
        u = (int(Y[j]) - vmin) // 2
        rowAt[cur[u]] = j
        cur[u] += 1
    pk = [None] * runp
    pstart = [10 ** 9] * (Wp + 2)
    w0 = [0, 0]
    for v in range(uneg, utop):
        st, L, p, b = seg[v], cnt[v], pofs[v], vmin + 2 * (v - K)
        if p < 0:
            continue
        Hfin = ((int(H[b]) << 8) if 0 <= b <= n else 0) | 8
        wfin = 0x4404 | (((60 * (-b) - 1) if b < 0 else 0) << 16)
        src = cnt[v + 8] if v + 8 < utop else 0
        if v + 2 < utop and pofs[v + 2] < 0:  # two-bin record: v and the absorbed v + 2
            b2 = b + 4
            Hfin = ((int(H[b2]) << 16) if b2 <= n else 0) | ((int(H[b]) << 8) if b <= n else 0) | 16
            wfin = 0x4104
            src |= (cnt[v + 10] if v + 10 < utop else 0) << 8
        if L == 0:
            w = max(0, (st - 1) >> 5)
            pk[p] = (0, src, Hfin, wfin)
            pstart[w] = min(pstart[w], p)
            if v - uneg < 2:
                w0[v - uneg] = w
            continue
        wa, wb = st >> 5, (st + L - 1) >> 5
        if v - uneg < 2:
            w0[v - uneg] = wa
        for w in range(wa, wb + 1):
            lo = max(st, 32 * w) - 32 * w
            hi = min(st + L, 32 * w + 32) - 32 * w
            mask = ((M32 if hi == 32 else (1 << hi) - 1) & (M32 << lo)) & M32
            pk[p] = (mask, src, Hfin, wfin) if w == wb else (mask, 0, 0, 0x4444)
            pstart[w] = min(pstart[w], p)
            p += 1
    cneg = sum(cnt[v] * 60 * (2 * K - (vmin + 2 * v)) for v in range(uneg))
    wins, htr, trl, z = [], [], [], []
    for q, np_ in ((0, n0), (1, n1)):
        a, zz = uneg + q, uneg + q + 2 * (np_ - 1)
        win = ht = tl = 0
        if np_ > 0:
            for i in range(4):
                if a + 2 * i <= zz:
                    win |= cnt[a + 2 * i] << (8 * i)
            for i in range(1, K + 1):
                b = vmin + 2 * (zz + 2 * i - K)
                if 0 <= b <= n:
                    ht |= int(H[b]) << (8 * (i - 1))
                if b < 0:
                    tl = 1
        wins.append(win)
        htr.append(ht)
        trl.append(tl)
        z.append(zz if np_ > 0 else -1)
    hwalk = 0
    for beta in range(U + 2 * K):
        b = vmin + 2 * (beta - K)
        Hb = int(H[b]) if 0 <= b <= n else 0
        zp = z[(beta - uneg) & 1]
        if Hb and beta >= uneg and zp >= 0 and beta <= zp + 2 * K:
            hwalk += Hb
    X = [[0] * n for _ in range(Wp)]
    B = (A * V[None, :]) == -1
    for p_, j in enumerate(rowAt):
        if j >= 0:
            for c in range(n):
                if B[j, c]:
                    X[p_ >> 5][c] |= 1 << (p_ & 31)
    return dict(pk=pk, pstart=pstart, w0=w0, win=wins, htr=htr, trl=trl, z=z, b1=pkb1, b2=runp, rneg=rneg,
                cneg=cneg, cabs=2 * m - hwalk - rtop - 8 * (utop - uneg), X=X, vmin=vmin, H=H, n=n)


def fitness(P, K, F):
    """eval_pk for one neighbour: deep rows, both walks record by record, trailing bins."""
    f, X, n = P["cabs"], P["X"], P["n"]
    a, b, c = (list(F) + [0, 0, 0])[:3]

    def planes(w):
        xa = X[w][a]
        xb = X[w][b] if K >= 2 else 0
        xc = X[w][c] if K == 3 else 0
        if K == 1:
            return xa, 0, 0
        if K == 2:
            return xa ^ xb, xa & xb, 0
        lo, hi = xa ^ xb ^ xc, (xa & xb) | (xc & (xa ^ xb))
        return lo, hi, lo & hi

    if P["rneg"] > 0:  # deep rows: cneg - 240 sum t
        st, nw = 0, (P["rneg"] + 31) // 32
        for w in range(nw):
            mask = ((1 << (P["rneg"] & 31)) - 1) if (w == nw - 1 and P["rneg"] & 31) else M32
            lo, hi, _ = planes(w)
            st += popc(lo & mask) + 2 * popc(hi & mask)
        f += P["cneg"] - 240 * st
    for q in range(2):
        pb, pe = (0, P["b1"]) if q == 0 else (P["b1"], P["b2"])
        if pb == pe:
            continue
        w_, pp, wd = P["win"][q], pb, P["w0"][q]
        while True:
            lo, hi, lh = planes(wd)
            pend = min(P["pstart"][wd + 1], pe)
            while pp < pend:
                r = P["pk"][pp]
                w_ = (w_ + 255 * popc(lo & r[0]) + 65535 * popc(hi & r[0]) + 16711425 * popc(lh & r[0])) & M32
                hb = prmt(w_, 0, r[3])
                fu = vabsdiff4_add(hb, r[2], dp2a_lo(r[3], hb, f & M32))
                f = fu if fu < 2 ** 31 else fu - 2 ** 32
                w_ = ((w_ | (r[1] << 32)) >> (r[2] & 31)) & M32  # funnel shift
                pp += 1
            if pend == pe:
                break
            wd += 1
        if not P["trl"][q]:
            f += sum(abs(((w_ >> (8 * i)) & 255) - ((P["htr"][q] >> (8 * i)) & 255)) for i in range(4))
        else:
            for i in range(K):
                h = (w_ >> (8 * i)) & 255
                bb = P["vmin"] + 2 * (P["z"][q] + 2 * (i + 1) - K)
                Hb = int(P["H"][bb]) if 0 <= bb <= n else 0
                f += (60 * (-bb) - 1 if bb < 0 else 0) * h + abs(h - Hb)
    return f


@pytest.mark.parametrize("pad", [0, 1])
def test_packed_model_matches_oracle(pad):
    rng = np.random.default_rng(11 + pad)
    checked = 0
    for trial in range(40):
        m, n, K = int(rng.integers(5, 160)), int(rng.integers(4, 80)), int(rng.integers(1, 4))
        inst = pi.planted_instance(m, n, int(rng.integers(1_000_000)))
        A = inst.A.astype(np.int64)
        kind = trial % 3  # random state (deep rows, empty points), near the secret, -secret (all negative)
        if kind == 0:
            V = np.where(rng.random(n) < 0.5, -1, 1).astype(np.int64)
        elif kind == 1:
            V = inst.secret.astype(np.int64).copy()
            V[rng.choice(n, 2, replace=False)] *= -1
        else:
            V = -inst.secret.astype(np.int64)
        P = build_plan(A, inst.S, V, K, pad)
        for _ in range(25):
            F = sorted(rng.choice(n, K, replace=False).tolist())
            V2 = V.copy()
            V2[F] *= -1
            assert fitness(P, K, F) == oracle.fitness(inst.A, inst.S, V2.astype(np.int8)), (m, n, K, F)
            checked += 1
    assert checked == 1000


def test_packed_model_absorbs_empty_points():
    """The two-bin records (absorbed empty points) are exercised: a sparse-value instance."""
    rng = np.random.default_rng(5)
    seen = 0
    for _ in range(30):
        m, n = 40, 61
        inst = pi.planted_instance(m, n, int(rng.integers(1_000_000)))
        V = np.where(rng.random(n) < 0.5, -1, 1).astype(np.int64)
        P = build_plan(inst.A.astype(np.int64), inst.S, V, 3, 1)
        seen += sum(1 for r in P["pk"] if r[3] == 0x4104)
        for _ in range(10):
            F = sorted(rng.choice(n, 3, replace=False).tolist())
            V2 = V.copy()
            V2[F] *= -1
            assert fitness(P, 3, F) == oracle.fitness(inst.A, inst.S, V2.astype(np.int8))
    assert seen > 0


def bytes_fit(A, S, V, K):
    """build_plan's guard for m > 255: every byte a walk window holds -- a walked
    bin's own rows plus those of the K points below it in its walk -- is <= 255, and so is H_b of
    every walked bin."""
    m, n = A.shape
    Y = A @ V
    H = np.bincount(S, minlength=n + 1)
    maxS = max(b for b in range(n + 1) if H[b] > 0)
    vmin = int(Y.min())
    U = (int(Y.max()) - vmin) // 2 + 1
    cnt = [int(((Y - vmin) // 2 == u).sum()) for u in range(U)]
    uneg = min(max((-2 * K - vmin + 1) >> 1, 0), U)
    utop = min(max(((maxS + 2 * K - vmin) >> 1) + 1, uneg), U)
    for v in range(uneg, utop + 2 * K):
        s4 = sum(cnt[v - 2 * t] for t in range(K + 1) if uneg <= v - 2 * t < utop)
        b = vmin + 2 * (v - K)
        if s4 > 255 or (0 <= b <= n and H[b] > 255):
            return False
    return True


@pytest.mark.parametrize("pad", [0, 1])
def test_packed_model_large_m_when_bytes_fit(pad):
    """m > 255: the byte-window arithmetic stays exact whenever the guard holds (random and
    near-secret states of planted instances up to 1024 rows); a state with > 255 rows on one
    lattice point fails the guard (the kernel then takes the segment plan)."""
    rng = np.random.default_rng(23 + pad)
    fit = 0
    for trial in range(8):
        m, n = [(300, int(rng.integers(20, 64))), (520, int(rng.integers(40, 64))),
                (1024, int(rng.integers(200, 260)))][trial % 3]
        K = int(rng.integers(1, 4))
        inst = pi.planted_instance(m, n, int(rng.integers(1_000_000)))
        A = inst.A.astype(np.int64)
        V = np.where(rng.random(n) < 0.5, -1, 1).astype(np.int64) if trial % 2 else inst.secret.astype(np.int64)
        if not bytes_fit(A, inst.S, V, K):
            continue
        fit += 1
        P = build_plan(A, inst.S, V, K, pad)
        for _ in range(6):
            F = sorted(rng.choice(n, K, replace=False).tolist())
            V2 = V.copy()
            V2[F] *= -1
            assert fitness(P, K, F) == oracle.fitness(inst.A, inst.S, V2.astype(np.int8)), (m, n, K, F)
    assert fit >= 5
    rows = np.tile(np.where(rng.random((1, 30)) < 0.5, -1, 1), (300, 1)).astype(np.int64)  # 300 equal rows
    V = rows[0].copy()  # every row at Y = 30: one walked lattice point of 300 rows
    assert not bytes_fit(rows, (rows @ V).astype(np.int32), V, 2)
