"""Seeded synthetic tridiagonal systems (shared by the CUDA path's tests/bench and the oracle).

This module holds NO solver arithmetic: it only draws coefficients from a
stateless counter hash so that every consumer (the oracle, the CUDA parity
tests, bench.py, every rank of a sharded run) sees bit-identical inputs for the
same (seed, global system index, row).

Recipe (SURVEY.md §8(d) "Concrete synthetic inputs"):

* ``h = splitmix64(seed ^ (array_id << 56) ^ global_row)`` with
  ``global_row = s * N + i`` for global system index ``s`` and row ``i``.
* fp32: the top 24 bits of ``h`` as a dyadic ``u`` in [0,1); fp64: the top 53.
  ``a, c, d = 2u - 1`` -- exact in the target precision, uniform on [-1, 1).
* ``a[0] = 0`` and ``c[N-1] = 0`` in every system (the ignored corner entries,
  DESIGN.md reading R3), then ``b = (|a| + |c|) + mu`` evaluated in the target
  precision (round-to-nearest, no FMA): strict row diagonal dominance with
  margin ``mu`` (default 1, the family the paper's solvers assume: no pivoting,
  PAPER.md §III-A, solves without pivoting).

Test-only families (never timed): ``poisson`` (tridiag(-1, 2, -1), the 1-D
Poisson matrix of the north_star's closed-form pin), ``const`` (tridiag(-1,
2+eps, -1)), ``adi`` (a = c = -r, b = 1 + 2r: the implicit diffusion step of
the ADI methods the paper's introduction names) and ``weak`` (dd with
a small margin).
"""
from __future__ import annotations

import numpy as np

__all__ = ["splitmix64", "uniform_pm1", "generate", "FAMILIES", "config_seed"]

_M64 = np.uint64(0xFFFFFFFFFFFFFFFF)
_GOLDEN = np.uint64(0x9E3779B97F4A7C15)
_MIX1 = np.uint64(0xBF58476D1CE4E5B9)
_MIX2 = np.uint64(0x94D049BB133111EB)

ARRAY_A, ARRAY_B, ARRAY_C, ARRAY_D = 0, 1, 2, 3

FAMILIES = ("dd", "poisson", "poisson_ones", "const", "adi", "weak")


def config_seed(config: int, dtype) -> int:
    """Seed convention of SURVEY.md §8(d): the config number, +100 for fp64 runs."""
    return int(config) + (100 if np.dtype(dtype) == np.float64 else 0)


def splitmix64(x: np.ndarray) -> np.ndarray:
    """Vigna's splitmix64 finaliser on uint64 arrays (wrap-around arithmetic)."""
    with np.errstate(over="ignore"):
        z = x + _GOLDEN
        z = (z ^ (z >> np.uint64(30))) * _MIX1
        z = (z ^ (z >> np.uint64(27))) * _MIX2
        return z ^ (z >> np.uint64(31))


def uniform_pm1(seed: int, array_id: int, rows: np.ndarray, dtype) -> np.ndarray:
    """Exact dyadic values in [-1, 1) for the given global row indices."""
    dtype = np.dtype(dtype)
    key = np.uint64(seed & 0xFFFFFFFFFFFFFFFF) ^ (np.uint64(array_id) << np.uint64(56))
    h = splitmix64(rows.astype(np.uint64) ^ key)
    if dtype == np.float32:
        u = (h >> np.uint64(40)).astype(np.int64)  # 24 bits
        return ((u - (1 << 23)).astype(np.float64) * 2.0 ** -23).astype(np.float32)
    if dtype == np.float64:
        u = (h >> np.uint64(11)).astype(np.int64)  # 53 bits
        return (u - (1 << 52)).astype(np.float64) * 2.0 ** -52
    raise ValueError(f"unsupported dtype {dtype}")


def generate(n: int, m: int, dtype=np.float32, seed: int = 1, family: str = "dd",
             first_system: int = 0, mu: float = 1.0, param: float = 0.5,
             chunk_rows: int = 1 << 22):
    """Return (a, b, c, d), each a C-contiguous (m, n) array of ``dtype``.

    ``first_system`` is the global index of the first system returned, so a rank
    owning systems [s0, s0+m) of a sharded batch draws exactly the rows an
    unsharded run would (global_row = s*N + i).
    """
    dtype = np.dtype(dtype)
    if family not in FAMILIES:
        raise ValueError(f"unknown family {family!r}")
    n, m = int(n), int(m)
    shape = (m, n)
    a = np.empty(shape, dtype)
    b = np.empty(shape, dtype)
    c = np.empty(shape, dtype)
    d = np.empty(shape, dtype)
    if m == 0 or n == 0:
        return a, b, c, d
    one = dtype.type(1)
    sys_per_chunk = max(1, chunk_rows // n)
    for s0 in range(0, m, sys_per_chunk):
        s1 = min(m, s0 + sys_per_chunk)
        g0 = (first_system + s0) * n
        rows = np.arange(g0, g0 + (s1 - s0) * n, dtype=np.uint64).reshape(s1 - s0, n)
        sl = slice(s0, s1)
        if family in ("dd", "weak"):
            a[sl] = uniform_pm1(seed, ARRAY_A, rows, dtype)
            c[sl] = uniform_pm1(seed, ARRAY_C, rows, dtype)
            d[sl] = uniform_pm1(seed, ARRAY_D, rows, dtype)
        else:
            if family in ("poisson", "poisson_ones", "const"):
                off = -one
            else:  # adi
                off = dtype.type(-param)
            a[sl] = off
            c[sl] = off
            if family == "poisson_ones":
                d[sl] = one
            else:
                d[sl] = uniform_pm1(seed, ARRAY_D, rows, dtype)
    a[:, 0] = 0
    c[:, n - 1] = 0
    if family in ("dd", "weak"):
        margin = dtype.type(mu if family == "dd" else param)  # weak: margin = param
        np.add(np.abs(a), np.abs(c), out=b)  # rounded in `dtype`
        b += margin
    elif family in ("poisson", "poisson_ones"):
        b[:] = dtype.type(2)
    elif family == "const":
        b[:] = dtype.type(2) + dtype.type(param)
    else:  # adi
        b[:] = one + dtype.type(2) * dtype.type(param)
    return a, b, c, d
