"""Per-solve time of config 1 (1 x 1024) and a 64 x 8192 batch: eager calls vs CUDA graph replay."""
import sys

import numpy as np
import torch

sys.path.insert(0, ".")
import paper_conf_ipps_davidsonzo11_b200 as tds  # noqa: E402
from paper_conf_ipps_davidsonzo11_b200 import inputs  # noqa: E402

for n, m in [(1024, 1), (8192, 64)]:
    plan = tds.Plan(n, m, "float32", device=0)
    plan.tune()
    a, b, c, d = (torch.from_numpy(v).cuda() for v in inputs.generate(n, m, np.float32, seed=1))
    x = torch.empty_like(d)
    ws = plan.workspace()
    s = torch.cuda.Stream()
    with torch.cuda.stream(s):
        for _ in range(10):
            tds.solve_batched(plan, a, b, c, d, out=x, workspace=ws)
        torch.cuda.synchronize()
        e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        e0.record()
        for _ in range(1000):
            tds.solve_batched(plan, a, b, c, d, out=x, workspace=ws)
        e1.record()
        torch.cuda.synchronize()
        eager = e0.elapsed_time(e1)
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
    print(f"{m} x {n}: eager {eager:.1f} us/solve, graph replay {e0.elapsed_time(e1):.1f} us/solve "
          f"(100 solves per graph)", flush=True)
