"""Config 1 (1 x 1024 fp32) and other launch-bound shapes: per-solve time of explicit on-chip plans under
CUDA-graph replay (100 solves per graph) vs eager back-to-back launches (diagnostic)."""
import sys

import numpy as np
import torch

sys.path.insert(0, ".")
import paper_conf_ipps_davidsonzo11_b200 as tds  # noqa: E402
from paper_conf_ipps_davidsonzo11_b200 import inputs  # noqa: E402


def per_solve(plan, a, b, c, d, x):
    ws = plan.workspace()
    s = torch.cuda.Stream()
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    with torch.cuda.stream(s):
        for _ in range(20):
            tds.solve_batched(plan, a, b, c, d, out=x, workspace=ws)
        torch.cuda.synchronize()
        e0.record()
        for _ in range(500):
            tds.solve_batched(plan, a, b, c, d, out=x, workspace=ws)
        e1.record()
        torch.cuda.synchronize()
        eager = e0.elapsed_time(e1) / 500 * 1e3
        g = torch.cuda.CUDAGraph()
    with torch.cuda.graph(g):
        for _ in range(100):
            tds.solve_batched(plan, a, b, c, d, out=x, workspace=ws)
    g.replay()
    torch.cuda.synchronize()
    e0.record()
    for _ in range(10):
        g.replay()
    e1.record()
    torch.cuda.synchronize()
    return eager, e0.elapsed_time(e1) / 1000 * 1e3


for n, m in [(1024, 1), (1024, 8), (4096, 1)]:
    a, b, c, d = (torch.from_numpy(v).cuda() for v in inputs.generate(n, m, np.float32, seed=1))
    x = torch.empty_like(d)
    cands = [("tuned", None)]
    for cl in range(0, 5):
        for tl in (0, 2, 4, 5):
            for T in (1, 8, 32):
                if tl == 5 and T != 1:
                    continue
                cands.append((f"c{cl} tl{tl} T{T}", dict(k_pass=[], cr_levels=cl, thomas_chains=T, tl_levels=tl,
                                                         cluster=1)))
    rows = []
    for name, p in cands:
        plan = tds.Plan(n, m, "float32", device=0)
        try:
            if p is None:
                plan.tune()
                name = (f"tuned (c{plan.info['cr_levels']} tl{plan.info['tl_levels']} T{plan.info['thomas_chains']} "
                        f"thr{plan.info['onchip_threads']})")
            else:
                plan.set_params(**p)
        except tds.TdsError:
            continue
        ea, gr = per_solve(plan, a, b, c, d, x)
        rows.append((gr, ea, name, plan.info["onchip_threads"]))
    rows.sort()
    for gr, ea, name, thr in rows[:12]:
        print(f"{m} x {n}: graph {gr:6.2f} us  eager {ea:6.2f} us  {name} threads {thr}", flush=True)
    print(flush=True)
