"""B200-native multi-stage batched tridiagonal solver (Davidson, Zhang & Owens, IPDPS 2011).

The compute path lives in ``libtds.so`` (csrc/, sm_100a CUDA + a C ABI declared
in include/tds.h).  This package is a thin ctypes binding over that library;
the native library is loaded lazily on first use and its absence is an error
(there is no CPU fallback).
"""
from . import inputs  # noqa: F401  (seeded generator; no solver arithmetic)

__all__ = ["inputs"]
