"""Time the tuned-shape plans of configs 3 (fp32, fp64) and 5 with the separate
x placement kernel vs the fused cluster placement (x_group), back-to-back
solves with CUDA events (diagnostic; bench.py is the measurement of record)."""
import sys

import numpy as np
import torch

sys.path.insert(0, ".")
import paper_conf_ipps_davidsonzo11_b200 as tds  # noqa: E402
from paper_conf_ipps_davidsonzo11_b200 import inputs  # noqa: E402
import oracle  # noqa: E402

CASES = [("cfg3 f32", 1 << 20, 16, np.float32, [7], 4), ("cfg3 f64", 1 << 20, 16, np.float64, [8], 3),
         ("cfg2 k3", 65536, 256, np.float32, [3], 4), ("cfg4 k1", 16384, 4096, np.float32, [1], 4)]


def timeit(fn, reps=50):
    for _ in range(5):
        fn()
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    torch.cuda.synchronize()
    e0.record()
    for _ in range(reps):
        fn()
    e1.record()
    torch.cuda.synchronize()
    return e0.elapsed_time(e1) / reps


for name, n, m, dt, kp, c in CASES:
    a, b, cc, d = inputs.generate(n, m, dt, seed=3)
    ta, tb, tc, td = (torch.from_numpy(v).cuda() for v in (a, b, cc, d))
    x = torch.empty_like(td)
    sdt = "float32" if dt == np.float32 else "float64"
    res = {}
    for G in (0, 2, 4, 8):
        plan = tds.Plan(n, m, sdt, device=0)
        try:
            plan.set_params(k_pass=kp, cr_levels=c, thomas_chains=16, cluster=1, tl_levels=5, x_group=G)
        except tds.TdsError as e:
            continue
        ws = plan.workspace()
        ms = timeit(lambda: tds.solve_batched(plan, ta, tb, tc, td, out=x, workspace=ws))
        xs = x.cpu().numpy()
        err = oracle.rel_err(xs[:2], oracle.thomas(a[:2], b[:2], cc[:2], d[:2]))
        res[G] = xs
        same = np.array_equal(xs, res[0]) if 0 in res else None
        print(f"{name} x_group={G}: {ms * 1e3:.1f} us/solve  {n * m / ms / 1e6:.1f} Geq/s  err={err:.2e} "
              f"bit-identical-to-unfused={same}", flush=True)
