"""Seeded synthetic inputs for the second binary fitness (UBQP).

Shared by the oracle side and the CUDA side like ``ppp_inputs``: instances and start vectors
from seeds, none of the method's arithmetic (no fitness, no neighbourhood, no tabu logic).

Recipe (the OR-Library / Beasley UBQP family: integer entries uniform in [-100, 100] at a given
density, symmetric):

* ``random_q(n, density, seed)``: numpy PCG64 stream seeded with ``seed``; the upper triangle
  (diagonal included) gets an entry with probability ``density``, uniform in [-100, 100];
  the lower triangle mirrors it;
* ``planted_ising(n, seed)``: a hidden sign vector z (uniform +-1); J = -z z^T (Ising energy
  s^T J s = -(s.z)^2, least at s = +-z) rewritten over x in {0,1} via s = 2x - 1 and
  x_i^2 = x_i: Q = 4 J - 4 diag(J 1); the constant 1^T J 1 is dropped;
* ``start_x(n, seed)``: uniform bits from a PCG64 stream seeded with ``seed``.
"""
from __future__ import annotations

import numpy as np


def random_q(n: int, density: float, seed: int) -> np.ndarray:
    rng = np.random.default_rng(seed)
    vals = rng.integers(-100, 101, size=(n, n), dtype=np.int64)
    keep = rng.random((n, n)) < density
    U = np.triu(np.where(keep, vals, 0))
    return (U + np.triu(U, 1).T).astype(np.int32)


def planted_ising(n: int, seed: int):
    """(Q, z): Q int32 n x n symmetric, z the hidden +-1 vector."""
    rng = np.random.default_rng(seed)
    z = rng.choice(np.array([-1, 1], dtype=np.int64), size=n)
    J = -np.outer(z, z)
    Q = 4 * J - 4 * np.diag(J.sum(axis=1))
    return Q.astype(np.int32), z


def start_x(n: int, seed: int) -> np.ndarray:
    rng = np.random.default_rng(seed)
    return rng.integers(0, 2, size=n, dtype=np.uint8)
