"""Interleaved vs system-major solve times (diagnostic; CUDA events)."""
import sys

import numpy as np
import torch

sys.path.insert(0, ".")
import paper_conf_ipps_davidsonzo11_b200 as tds  # noqa: E402
from paper_conf_ipps_davidsonzo11_b200 import inputs  # noqa: E402


def timeit(fn, reps=30):
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


for name, n, m in [("cfg4 shape", 16384, 4096), ("cfg2 shape", 65536, 256), ("cfg3 shape", 1 << 20, 16),
                   ("ADI 1024^2", 1024, 1024)]:
    a, b, c, d = inputs.generate(n, m, np.float32, seed=1)
    plan = tds.Plan(n, m, "float32", device=0)
    plan.tune()
    ts = [torch.from_numpy(v).cuda() for v in (a, b, c, d)]
    ti = [t.t().contiguous() for t in ts]
    x = torch.empty_like(ts[3])
    xi = torch.empty_like(ti[3])
    ws = plan.workspace()
    wi = torch.empty(plan.interleaved_workspace_bytes, dtype=torch.uint8, device="cuda")
    us_s = timeit(lambda: tds.solve_batched(plan, *ts, out=x, workspace=ws))
    us_i = timeit(lambda: tds.solve_interleaved(plan, *ti, out=xi, workspace=wi))
    eq = n * m
    print(f"{name} ({m} x {n}): system-major {us_s:.1f} us ({eq / us_s / 1e3:.1f} Geq/s), "
          f"interleaved {us_i:.1f} us ({eq / us_i / 1e3:.1f} Geq/s); transposes move "
          f"{(32 + 8) * eq / 1e6:.0f} MB -> {(32 + 8) * eq / (us_i - us_s) / 1e3:.0f} GB/s", flush=True)
