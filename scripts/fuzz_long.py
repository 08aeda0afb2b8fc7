"""Long randomized plan fuzz (diagnostic; the test suite runs a seeded 320-draw
subset): random n, m, dtype and plan parameters, every plan the planner
accepts solved on the GPU and checked against the oracle.

    python scripts/fuzz_long.py [draws] [seed] [cv]

With "cv" every draw is a plan of the paper's coalesced load variant
(strided = 2: one pass of log2(32 / sizeof(T)) .. 4 levels, random T,
random ragged n on a 16-byte batch stride, chunking).
"""
import sys

import numpy as np
import torch

sys.path.insert(0, ".")
import oracle  # noqa: E402
import paper_conf_ipps_davidsonzo11_b200 as tds  # noqa: E402
from paper_conf_ipps_davidsonzo11_b200 import inputs  # noqa: E402

draws = int(sys.argv[1]) if len(sys.argv) > 1 else 2000
rng = np.random.default_rng(int(sys.argv[2]) if len(sys.argv) > 2 else 7)
CV_ONLY = len(sys.argv) > 3 and sys.argv[3] == "cv"
ran = bad = inter = coupled = cv = 0
for i in range(draws):
    dtype = np.float32 if rng.random() < 0.7 else np.float64
    n = int(rng.choice([rng.integers(1, 5000), rng.integers(5000, 400000), 1 << int(rng.integers(10, 20))]))
    m = int(rng.integers(1, 9))
    k = int(rng.integers(0, 13))
    passes = 0 if k == 0 else int(rng.integers(1, min(3, k) + 1))
    kp = [] if k == 0 else [k // passes + (1 if j < k % passes else 0) for j in range(passes)]
    c_lv = int(rng.integers(0, 5 if dtype == np.float32 else 4))
    params = dict(k_pass=kp, cr_levels=c_lv, thomas_chains=int(2 ** rng.integers(0, 7)),
                  cluster=int(rng.choice([1, 1, 1, 2, 4, 8, 16])), tl_levels=int(rng.choice([0, 1, 2, 3, 5])),
                  x_group=int(rng.choice([0, 0, 0, 2, 4, 8])), strided=int(rng.choice([0, 0, 1, 2])),
                  split_threads=int(rng.choice([128, 256, 512])), split_tile_rows=int(rng.choice([2048, 4096, 8192])),
                  theta=int(rng.choice([1, 16, 148, 4736])), chunk_systems=int(rng.choice([0, 0, 1, 2, 3])))
    stride = 0
    if CV_ONLY:
        g = 3 if dtype == np.float32 else 2
        params = dict(k_pass=[int(rng.integers(g, 5))], cr_levels=0, tl_levels=0, cluster=1, strided=2,
                      thomas_chains=int(2 ** rng.integers(0, 9 if dtype == np.float64 else 8)),
                      chunk_systems=int(rng.choice([0, 0, 1, 2, 3])))
        e = 16 // np.dtype(dtype).itemsize
        stride = -(-n // e) * e
    if params["strided"] == 2:  # the coalesced variant: PCR-Thomas without register / thread CR levels
        params.update(cr_levels=0, tl_levels=0)
    plan = tds.Plan(n, m, "float32" if dtype == np.float32 else "float64", device=0, batch_stride=stride)
    try:
        plan.set_params(**params)
    except tds.TdsError:
        continue
    # fp64 draws: half of them on long-range-coupled families (Poisson, tridiag(-1, 2 + 1e-6, -1)) with
    # 10 kappa eps tolerances -- random plans must carry the coupling, not only the dd-random data
    fam = "dd"
    if dtype == np.float64 and rng.random() < 0.5:
        fam = "poisson" if rng.random() < 0.5 else "const"
    kw = {"param": 1e-6} if fam == "const" else {}
    a, b, c, d = inputs.generate(n, m, dtype, seed=5000 + i, family=fam, **kw)
    if stride and stride != n:  # padded batch stride (the coalesced variant needs 16-byte system starts)
        pad = lambda v: torch.from_numpy(np.pad(v, ((0, 0), (0, stride - n)), constant_values=1.0)).cuda()
        x = tds.solve_batched(plan, *[pad(v) for v in (a, b, c, d)])
        torch.cuda.synchronize()
        x = np.ascontiguousarray(x.cpu().numpy().reshape(m, stride)[:, :n])
    else:
        x = tds.solve_batched(plan, *[torch.from_numpy(v).cuda() for v in (a, b, c, d)])
        torch.cuda.synchronize()
        x = x.cpu().numpy()
    err = oracle.rel_err(x, oracle.thomas(a, b, c, d))
    if fam == "dd":
        tol = 1e-4 if dtype == np.float32 else 1e-10
    else:
        delta = kw.get("param", 0.0)
        cs = np.cos(np.pi / (n + 1))
        tol = 10 * (2 + delta + 2 * cs) / max(2 + delta - 2 * cs, 1e-300) * 2.22e-16
        coupled += 1
    ok = np.all(np.isfinite(x)) and err <= tol
    if ok and plan.info["batch_stride"] == n and rng.random() < 0.3:  # the interleaved layout: bit-identical
        xi = tds.solve_interleaved(plan, *[torch.from_numpy(np.ascontiguousarray(v.T)).cuda() for v in (a, b, c, d)])
        torch.cuda.synchronize()
        ok = bool(np.array_equal(xi.cpu().numpy().T, x))
        inter += 1
    ran += 1
    cv += plan.info["strided"] == 2
    if not ok:
        bad += 1
        print(f"BAD draw {i}: {dtype.__name__} {fam} n={n} m={m} {params} err={err:.3e}", flush=True)
print(f"fuzz: {ran} plans run ({inter} also through the interleaved layout, {coupled} on coupled fp64 "
      f"families, {cv} coalesced-variant plans), {bad} bad", flush=True)
sys.exit(1 if bad else 0)
