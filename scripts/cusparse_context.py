"""Context comparison: cuSPARSE's batched tridiagonal
solvers on the same B200, the same BASELINE.json workloads and the same
generated systems as bench.py -- a library point of reference, not the paper's
comparison system and not a target.

    python scripts/cusparse_context.py [--configs 2 3 4] [--reps 20]

For each config: cusparseSgtsv2StridedBatch (CR + PCR, no pivoting -- the
same algorithm family as the paper's) and, for one huge system per call,
cusparseSgtsv2_nopivot looped over the batch; tds with the STATIC and TUNED
plans on the same device buffers.  Device time by CUDA events on the launching
stream, median of --reps after 3 warm-ups.  cuSPARSE overwrites the right-hand
side in place, so every timed call copies d first; that copy (8 B/eq) is timed
separately and subtracted.  Prints one JSON line per (config, solver), each
with the solver's relative residual against A x = d (fp64, on the host, on a
sample of systems).
"""
from __future__ import annotations

import argparse
import ctypes
import json
import os
import sys

import numpy as np
import torch

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
import paper_conf_ipps_davidsonzo11_b200 as tds  # noqa: E402

CONFIGS = {1: (1024, 1), 2: (65536, 256), 3: (1 << 20, 16), 4: (16384, 4096)}


def load_cusparse():
    import nvidia.cusparse
    path = os.path.join(os.path.dirname(nvidia.cusparse.__file__), "lib", "libcusparse.so.12")
    lib = ctypes.CDLL(path)
    vp, i32, sz = ctypes.c_void_p, ctypes.c_int, ctypes.c_size_t
    lib.cusparseCreate.argtypes = [ctypes.POINTER(vp)]
    lib.cusparseSetStream.argtypes = [vp, vp]
    lib.cusparseSgtsv2StridedBatch_bufferSizeExt.argtypes = [vp, i32, vp, vp, vp, vp, i32, i32,
                                                             ctypes.POINTER(sz)]
    lib.cusparseSgtsv2StridedBatch.argtypes = [vp, i32, vp, vp, vp, vp, i32, i32, vp]
    lib.cusparseSgtsv2_nopivot_bufferSizeExt.argtypes = [vp, i32, i32, vp, vp, vp, vp, i32, ctypes.POINTER(sz)]
    lib.cusparseSgtsv2_nopivot.argtypes = [vp, i32, i32, vp, vp, vp, vp, i32, vp]
    return lib


def check(st, what):
    if st != 0:
        raise RuntimeError(f"{what}: cusparse status {st}")


def residual_sample(a, b, c, d, x, rows):
    """max over sampled systems of ||Ax - d||_inf / ||d||_inf, fp64 on the host."""
    worst = 0.0
    for s in rows:
        A, B, C, D, X = (t[s].double().cpu().numpy() for t in (a, b, c, d, x))
        r = B * X - D
        r[1:] += A[1:] * X[:-1]
        r[:-1] += C[:-1] * X[1:]
        worst = max(worst, float(np.abs(r).max() / np.abs(D).max()))
    return worst


def timed(fn, reps):
    s = torch.cuda.current_stream()
    for _ in range(3):
        fn()
    ts = []
    for _ in range(reps):
        e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        e0.record(s)
        fn()
        e1.record(s)
        e1.synchronize()
        ts.append(e0.elapsed_time(e1))
    ts.sort()
    return ts[len(ts) // 2]


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--configs", type=int, nargs="*", default=[2, 3, 4])
    ap.add_argument("--reps", type=int, default=20)
    args = ap.parse_args()
    lib = load_cusparse()
    h = ctypes.c_void_p()
    check(lib.cusparseCreate(ctypes.byref(h)), "create")
    check(lib.cusparseSetStream(h, ctypes.c_void_p(torch.cuda.current_stream().cuda_stream)), "stream")
    dev = torch.device("cuda:0")
    for cfg in args.configs:
        n, m = CONFIGS[cfg]
        a, b, c, d = (torch.from_numpy(v).to(dev) for v in tds.inputs.generate(n, m, np.float32, seed=cfg))
        eqs = n * m
        sample = sorted(set([0, m // 2, m - 1]))
        x = torch.empty_like(d)
        t_copy = timed(lambda: x.copy_(d), args.reps)

        def out(solver, ms, res, note=""):
            print(json.dumps({"config": cfg, "n": n, "m": m, "solver": solver, "ms": ms,
                              "eq_per_s": eqs / (ms * 1e-3), "residual": res, "note": note}), flush=True)

        # gtsv2StridedBatch: CR + PCR, no pivoting
        bs = ctypes.c_size_t()
        st = lib.cusparseSgtsv2StridedBatch_bufferSizeExt(h, n, a.data_ptr(), b.data_ptr(), c.data_ptr(),
                                                          x.data_ptr(), m, n, ctypes.byref(bs))
        if st == 0:
            buf = torch.empty(max(bs.value, 1), dtype=torch.uint8, device=dev)

            def sb():
                x.copy_(d)
                check(lib.cusparseSgtsv2StridedBatch(h, n, a.data_ptr(), b.data_ptr(), c.data_ptr(), x.data_ptr(),
                                                     m, n, buf.data_ptr()), "gtsv2StridedBatch")
            ms = timed(sb, args.reps) - t_copy
            torch.cuda.synchronize()
            out("cusparseSgtsv2StridedBatch", ms, residual_sample(a, b, c, d, x, sample),
                f"d->x copy ({t_copy:.4f} ms) subtracted")
            del buf
        else:
            out("cusparseSgtsv2StridedBatch", None, None, f"bufferSize status {st}")

        # gtsv2_nopivot: one call per system (the library's large-system solver)
        bs = ctypes.c_size_t()
        st = lib.cusparseSgtsv2_nopivot_bufferSizeExt(h, n, 1, a.data_ptr(), b.data_ptr(), c.data_ptr(),
                                                      x.data_ptr(), n, ctypes.byref(bs))
        if st == 0 and m <= 256:
            buf = torch.empty(max(bs.value, 1), dtype=torch.uint8, device=dev)

            def nop():
                x.copy_(d)
                for s in range(m):
                    o = s * n * 4
                    check(lib.cusparseSgtsv2_nopivot(h, n, 1, a.data_ptr() + o, b.data_ptr() + o,
                                                     c.data_ptr() + o, x.data_ptr() + o, n, buf.data_ptr()),
                          "gtsv2_nopivot")
            ms = timed(nop, max(3, args.reps // 4)) - t_copy
            torch.cuda.synchronize()
            out("cusparseSgtsv2_nopivot (loop over systems)", ms, residual_sample(a, b, c, d, x, sample),
                f"{m} calls; d->x copy subtracted")
            del buf

        # tds, static and tuned plans, same buffers
        for mode in ("static", "tuned"):
            plan = tds.Plan(n, m, "float32", device=0, mode="static")
            if mode == "tuned":
                plan.tune()
            ws = plan.workspace()
            ms = timed(lambda: tds.solve_batched(plan, a, b, c, d, out=x, workspace=ws), args.reps)
            torch.cuda.synchronize()
            out(f"tds ({mode})", ms, residual_sample(a, b, c, d, x, sample),
                json.dumps({k: v for k, v in plan.info.items() if k in ("k", "k_pass", "n_sub", "cluster")}))
        del a, b, c, d, x
        torch.cuda.empty_cache()


if __name__ == "__main__":
    main()
