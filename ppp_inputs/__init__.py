"""Seeded synthetic inputs for the PPP tabu-search hot path.

This module is the ONE piece shared by the oracle side (``oracle/``) and the CUDA side
(``paper_conf_ipps_luongmt10_b200``): it produces instances and start vectors from seeds.
It contains none of the method's arithmetic (no fitness, no neighbourhood, no tabu logic);
it only draws random bits and plants a secret, as the instance recipe of DESIGN.md §3 says.

Recipe (reading R13, BASELINE.json ``north_star``; PAPER.md:81-84 and 249-250 only
cite Pointcheval [8] / Knudsen-Meier [10] instances, which are not published):

* one splitmix64 stream seeded with ``instance_seed``;
* A (m x n, entries +-1) is filled row-major, 64 entries per draw, least significant bit
  first, bit 1 -> -1;
* the planted secret V* takes ceil(n/64) further draws (same bit convention);
* y = A V*; every row j with y_j < 0 is negated, so A V* >= 0 (rows with y_j = 0 are kept);
* S = {y_j} is the multiset of Definition 1.

Start vectors: V0 takes ceil(n/64) draws from a second stream seeded with ``seed``.
Restart r of a batch uses ``restart_seed(seed, r)`` = first draw of a stream seeded with
``seed + r`` (reading R12).
"""
from __future__ import annotations

import dataclasses

import numpy as np

MASK64 = (1 << 64) - 1
GOLDEN = 0x9E3779B97F4A7C15


def splitmix64_stream(state: int):
    """Infinite generator of splitmix64 outputs (Steele, Lea & Flood 2014).

    Each draw: s += 0x9E3779B97F4A7C15; z = s; z = (z ^ z>>30) * 0xBF58476D1CE4E5B9;
    z = (z ^ z>>27) * 0x94D049BB133111EB; return z ^ z>>31 (all mod 2^64).
    """
    s = state & MASK64
    while True:
        s = (s + GOLDEN) & MASK64
        z = s
        z = ((z ^ (z >> 30)) * 0xBF58476D1CE4E5B9) & MASK64
        z = ((z ^ (z >> 27)) * 0x94D049BB133111EB) & MASK64
        yield z ^ (z >> 31)


def _draw_pm1(gen, count: int) -> np.ndarray:
    """`count` +-1 entries, 64 per draw, LSB first, bit 1 -> -1."""
    ndraw = (count + 63) // 64
    words = np.array([next(gen) for _ in range(ndraw)], dtype=np.uint64)
    bits = np.unpackbits(words.view(np.uint8), bitorder="little")[:count]
    return (1 - 2 * bits.astype(np.int8)).astype(np.int8)


def restart_seed(seed: int, r: int) -> int:
    """Seed of restart r: the first splitmix64 output of a stream seeded with seed + r."""
    return next(splitmix64_stream((seed + r) & MASK64))


def start_vector(n: int, seed: int) -> np.ndarray:
    """V0 in {+-1}^n from a splitmix64 stream seeded with `seed` (ceil(n/64) draws)."""
    return _draw_pm1(splitmix64_stream(seed), n)


@dataclasses.dataclass(frozen=True)
class Instance:
    """A planted PPP instance (Definition 1)."""

    A: np.ndarray  # (m, n) int8, entries +-1, row-major
    S: np.ndarray  # (m,) int32, the multiset, non-negative
    secret: np.ndarray  # (n,) int8, the planted V* (A V* is a permutation of S)
    seed: int

    @property
    def m(self) -> int:
        return int(self.A.shape[0])

    @property
    def n(self) -> int:
        return int(self.A.shape[1])


def planted_instance(m: int, n: int, instance_seed: int) -> Instance:
    """Pointcheval-style planted instance, recipe in the module docstring."""
    if m < 1 or n < 1:
        raise ValueError("m and n must be >= 1")
    gen = splitmix64_stream(instance_seed)
    A = _draw_pm1(gen, m * n).reshape(m, n).copy()
    secret = _draw_pm1(gen, n)
    y = A.astype(np.int64) @ secret.astype(np.int64)
    neg = y < 0
    A[neg] = -A[neg]
    y[neg] = -y[neg]
    return Instance(A=A, S=y.astype(np.int32), secret=secret, seed=instance_seed)


# The five configurations of BASELINE.json (C1..C5) with the seeds of DESIGN.md §3.
# (m, n, k, iters); instance_seed = 1000 + cfg#, run seed = 1 + cfg#.
CONFIGS = {
    "C1": dict(m=21, n=21, k=1, iters=1000),
    "C2": dict(m=73, n=73, k=2, iters=10000),
    "C3": dict(m=81, n=81, k=3, iters=10000),
    "C4": dict(m=101, n=117, k=3, iters=2000),
    "C5": dict(m=1024, n=1024, k=3, iters=10),
}


def config_instance(name: str) -> Instance:
    c = CONFIGS[name]
    return planted_instance(c["m"], c["n"], 1000 + int(name[1:]))


def config_seed(name: str) -> int:
    return 1 + int(name[1:])


def default_tenure(n: int, k: int) -> int:
    """floor(C(n,k)/6): "tabu list size ... m/6 where m is the number of neighbors"
    (reading R3)."""
    from math import comb

    return comb(n, k) // 6
