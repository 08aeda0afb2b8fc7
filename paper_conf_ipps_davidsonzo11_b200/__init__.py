"""B200-native multi-stage batched tridiagonal solver (Davidson, Zhang & Owens, IPDPS 2011).

The compute path lives in ``libtds.so`` (csrc/: sm_100a CUDA kernels and the C
ABI declared in include/tds.h).  This package is a thin ctypes binding with the
same names; the native library is loaded on first use and its absence is an
error (there is no CPU fallback).
"""
from . import inputs  # noqa: F401  (seeded generator; no solver arithmetic)
from ._lib import TdsError  # noqa: F401
from .api import Plan, device_props, generate, solve_batched, solve_interleaved, split_batched, version  # noqa: F401

__all__ = ["Plan", "solve_batched", "solve_interleaved", "split_batched", "generate", "device_props", "version",
           "TdsError", "inputs"]
