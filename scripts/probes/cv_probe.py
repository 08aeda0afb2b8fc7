"""The paper's two base-kernel load variants against the
de-interleaved path at the same k: strided = 1 (strided gather), strided = 2
(coalesced sector groups, rows beyond shared memory in the workspace), and the
tuned plan (diagnostic; back-to-back solves, CUDA events)."""
import sys

import numpy as np
import torch

sys.path.insert(0, ".")
import paper_conf_ipps_davidsonzo11_b200 as tds  # noqa: E402
from paper_conf_ipps_davidsonzo11_b200 import inputs  # noqa: E402


def timeit(fn, reps=20):
    for _ in range(3):
        fn()
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    torch.cuda.synchronize()
    e0.record()
    for _ in range(reps):
        fn()
    e1.record()
    torch.cuda.synchronize()
    return e0.elapsed_time(e1) / reps * 1e3


SHAPES = [("cfg2 256 x 65536", 65536, 256, np.float32, (3, 4)), ("cfg4 4096 x 16384", 16384, 4096, np.float32, (3, 4)),
          ("cfg3 16 x 2^20", 1 << 20, 16, np.float32, (4,)), ("16384 x 2048", 2048, 16384, np.float32, (3, 4)),
          ("65536 x 512", 512, 65536, np.float32, (3, 4)), ("f64 256 x 65536", 65536, 256, np.float64, (2, 4))]
for name, n, m, dt, ks in SHAPES:
    dts = "float32" if dt == np.float32 else "float64"
    c_lv = 4 if dt == np.float32 else 3
    a, b, c, d = (torch.from_numpy(v).cuda() for v in inputs.generate(n, m, dt, seed=1))
    x = torch.empty_like(d)
    for k in ks:
        rows = []
        for sv, T in [(0, 1), (1, 1), (2, 16), (2, 32), (2, 64), (2, 128)]:
            plan = tds.Plan(n, m, dts, device=0)
            try:
                if sv == 2:
                    plan.set_params(k_pass=[k], cr_levels=0, thomas_chains=T, cluster=1, tl_levels=0, strided=2)
                else:
                    plan.set_params(k_pass=[k], cr_levels=c_lv, thomas_chains=1, cluster=1, tl_levels=5, strided=sv)
            except tds.TdsError as e:
                rows.append(f"strided={sv} T={T}: rejected ({e})")
                continue
            ws = plan.workspace()
            us = timeit(lambda: tds.solve_batched(plan, a, b, c, d, out=x, workspace=ws))
            rows.append(f"strided={sv} T={T}: {us:.1f} us ({n * m / us / 1e3:.1f} Geq/s)")
        for r in rows:
            print(f"{name} k={k} {r}", flush=True)
    plan = tds.Plan(n, m, dts, device=0)
    plan.tune()
    ws = plan.workspace()
    us = timeit(lambda: tds.solve_batched(plan, a, b, c, d, out=x, workspace=ws))
    i = plan.info
    print(f"{name} tuned (k_pass {i['k_pass']}, cluster {i['cluster']}, strided {i['strided']}, T {i['thomas_chains']},"
          f" trials {plan.tune_trials if hasattr(plan, 'tune_trials') else '?'}): {us:.1f} us", flush=True)
