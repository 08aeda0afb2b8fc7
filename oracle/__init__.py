"""CPU oracle for the multi-stage tridiagonal solver.  TEST INFRASTRUCTURE ONLY.

Only ``tests/``, ``__graft_entry__.smoke()`` and ``bench.py``'s cpu_baseline /
``--impl reference`` legs may import this package.  It shares no code with the
CUDA path (``paper_conf_ipps_davidsonzo11_b200``): not a kernel, header, helper,
table or constant generator.  The only shared module is the seeded input
generator ``paper_conf_ipps_davidsonzo11_b200.inputs`` (no solver arithmetic).

Contents (each cites the passage it follows; PAPER.md = /root/reference/PAPER.md):

* ``thomas``      -- fp64 Thomas solve (C, ``oracle/thomas.c``): the plain
                     definition the method must reproduce (§III-A
                     P:L269-273, stage 4 P:L511-512; textbook form).
* ``pcr_split``   -- k textbook PCR levels in fp64 (PAPER.md P:L199-200 cites
                     Hockney & Jesshope [11]; Fig. 3a), the
                     definition the split stage (Stages 1-2, §III-B/C
                     P:L296-303) follows.
* ``permutation`` -- the canonical subsystem order after k levels (Fig. 3a
                     P:L386-394: 2 systems of 4, 4 of 2, 8 of 1).
* ``residual`` / ``backward_error`` / ``rel_err`` -- fp64 error metrics.
* ``plan``        -- the reference planner (``oracle/plan.py``): the method's integers of
                     §IV-B/C (on-chip entry size, k, passes, T, theta, segments).

Parity status: every function here is pinned by ``tests/test_oracle.py``
against something other than itself (dense Gaussian elimination, LAPACK
``dgtsv``, closed forms of the Poisson matrix, exact dyadic PCR values,
brute-force orderings, the paper's printed parameter values).
"""
from __future__ import annotations

import ctypes
import os
import subprocess

import numpy as np

from . import plan  # noqa: F401  (reference planner)

_HERE = os.path.dirname(os.path.abspath(__file__))
_LIB_PATH = os.path.join(_HERE, "liboracle.so")
_lib = None


def build(force: bool = False) -> str:
    """Compile oracle/thomas.c with gcc (-O2 -ffp-contract=off -fopenmp)."""
    src = os.path.join(_HERE, "thomas.c")
    if force or not os.path.exists(_LIB_PATH) or os.path.getmtime(_LIB_PATH) < os.path.getmtime(src):
        tmp = _LIB_PATH + f".tmp{os.getpid()}"
        subprocess.check_call(["gcc", "-O2", "-ffp-contract=off", "-fopenmp", "-fPIC", "-shared",
                               "-o", tmp, src])
        os.replace(tmp, _LIB_PATH)
    return _LIB_PATH


def _load():
    global _lib
    if _lib is None:
        build()
        lib = ctypes.CDLL(_LIB_PATH)
        lib.oracle_thomas_f64.restype = ctypes.c_int
        lib.oracle_thomas_f64.argtypes = [ctypes.c_int64, ctypes.c_int64, ctypes.c_int64] + \
            [ctypes.c_void_p] * 5 + [ctypes.c_int]
        lib.oracle_num_threads.restype = ctypes.c_int
        _lib = lib
    return _lib


def num_threads() -> int:
    return int(_load().oracle_num_threads())


def _as2d64(x):
    x = np.asarray(x)
    if x.ndim == 1:
        x = x[None, :]
    return np.ascontiguousarray(x, dtype=np.float64)  # exact upcast from fp32


def thomas(a, b, c, d, threads: int = 0) -> np.ndarray:
    """fp64 Thomas solve of each row-system of (m, n) arrays; returns x (m, n) fp64.

    ``a[:, 0]`` and ``c[:, n-1]`` are ignored (reading R3).
    """
    squeeze = np.asarray(d).ndim == 1
    a, b, c, d = (_as2d64(v) for v in (a, b, c, d))
    m, n = d.shape
    x = np.empty((m, n), np.float64)
    if m == 0:
        return x
    rc = _load().oracle_thomas_f64(n, m, n, a.ctypes.data, b.ctypes.data, c.ctypes.data,
                                   d.ctypes.data, x.ctypes.data, int(threads))
    if rc != 0:
        raise RuntimeError(f"oracle_thomas_f64 failed ({rc})")
    return x[0] if squeeze else x


def pcr_split(a, b, c, d, k: int):
    """Apply k textbook PCR levels (fp64, unnormalised) to every system.

    Level with stride s = 2^(j-1) (Hockney & Jesshope [11], cited P:L199-200):
        k1 = a_i / b_{i-s},   k2 = c_i / b_{i+s}
        a'_i = -a_{i-s} k1
        b'_i = b_i - c_{i-s} k1 - a_{i+s} k2
        c'_i = -c_{i+s} k2
        d'_i = d_i - d_{i-s} k1 - d_{i+s} k2
    Rows outside [0, n) are identity rows (a, b, c, d) = (0, 1, 0, 0)
    (reading R2).  Returns (a', b', c', d') in ORIGINAL row order;
    rows congruent to r mod 2^k then form independent tridiagonal systems with
    coupling stride 2^k (Fig. 3a).
    """
    a, b, c, d = (_as2d64(v).copy() for v in (a, b, c, d))
    m, n = d.shape
    a[:, 0] = 0.0
    c[:, n - 1] = 0.0
    for j in range(int(k)):
        s = 1 << j
        if s >= n:
            break
        al = np.zeros_like(a); bl = np.ones_like(b); cl = np.zeros_like(c); dl = np.zeros_like(d)
        ar = np.zeros_like(a); br = np.ones_like(b); cr = np.zeros_like(c); dr = np.zeros_like(d)
        al[:, s:], bl[:, s:], cl[:, s:], dl[:, s:] = a[:, :-s], b[:, :-s], c[:, :-s], d[:, :-s]
        ar[:, :-s], br[:, :-s], cr[:, :-s], dr[:, :-s] = a[:, s:], b[:, s:], c[:, s:], d[:, s:]
        k1 = a / bl
        k2 = c / br
        a, b, c, d = (-al * k1,
                      b - cl * k1 - ar * k2,
                      -cr * k2,
                      d - dl * k1 - dr * k2)
    return a, b, c, d


def permutation(n: int, k: int) -> np.ndarray:
    """Canonical subsystem order after k levels (reading R5).

    perm[off(r) + j] = r + 2^k j for residues r = 0..min(2^k, n)-1 ascending,
    j ascending; n_r = ceil((n - r) / 2^k), off(r) = sum_{r' < r} n_r'.
    """
    step = 1 << int(k)
    return np.concatenate([np.arange(r, n, step, dtype=np.int64) for r in range(min(step, n))])


def subsystem(a, b, c, d, k: int, r: int):
    """The residue-r subsystem (rows r, r+2^k, ...) of already-split arrays."""
    step = 1 << int(k)
    return tuple(np.ascontiguousarray(v[..., r::step]) for v in (a, b, c, d))


def matvec(a, b, c, x):
    """y = A x for the tridiagonal A (fp64), a[:,0] and c[:,n-1] ignored."""
    a, b, c, x = (_as2d64(v) for v in (a, b, c, x))
    y = b * x
    y[:, 1:] += a[:, 1:] * x[:, :-1]
    y[:, :-1] += c[:, :-1] * x[:, 1:]
    return y


def residual(a, b, c, d, x) -> float:
    """max over systems of ||A x - d||_inf / ||d||_inf (north_star residual)."""
    d64 = _as2d64(d)
    r = np.abs(matvec(a, b, c, x) - d64).max(axis=1)
    dn = np.abs(d64).max(axis=1)
    dn[dn == 0] = 1.0
    return float((r / dn).max()) if r.size else 0.0


def backward_error(a, b, c, d, x) -> float:
    """max over systems of ||Ax-d||_inf / (||A||_inf ||x||_inf + ||d||_inf)."""
    a64, b64, c64, d64, x64 = (_as2d64(v) for v in (a, b, c, d, x))
    a64 = a64.copy(); c64 = c64.copy()
    a64[:, 0] = 0; c64[:, -1] = 0
    r = np.abs(matvec(a64, b64, c64, x64) - d64).max(axis=1)
    an = (np.abs(a64) + np.abs(b64) + np.abs(c64)).max(axis=1)
    den = an * np.abs(x64).max(axis=1) + np.abs(d64).max(axis=1)
    den[den == 0] = 1.0
    return float((r / den).max()) if r.size else 0.0


def rel_err(x, xref) -> float:
    """Normwise relative error ||x - xref||_inf / ||xref||_inf per system, max over systems."""
    x = _as2d64(x); xref = _as2d64(xref)
    num = np.abs(x - xref).max(axis=1)
    den = np.abs(xref).max(axis=1)
    den[den == 0] = 1.0
    return float((num / den).max()) if num.size else 0.0
