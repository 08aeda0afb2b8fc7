"""Config 3 (16 x 2^20 fp32): L2-resident chunks x split schedules (diagnostic).
A chunk's split output (12 B/row per pass) stays in the 126 MB L2 when
chunk_systems is small, so a second split pass and the on-chip loads can hit L2."""
import sys

import numpy as np
import torch

sys.path.insert(0, ".")
import paper_conf_ipps_davidsonzo11_b200 as tds  # noqa: E402
from paper_conf_ipps_davidsonzo11_b200 import inputs  # noqa: E402

n, m = 1 << 20, 16
a, b, c, d = inputs.generate(n, m, np.float32, seed=3)
ta, tb, tc, td = (torch.from_numpy(v).cuda() for v in (a, b, c, d))
x = torch.empty_like(td)


def timeit(fn, reps=40):
    for _ in range(5):
        fn()
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    torch.cuda.synchronize()
    e0.record()
    for _ in range(reps):
        fn()
    e1.record()
    torch.cuda.synchronize()
    return e0.elapsed_time(e1) / reps * 1e3


base = dict(cr_levels=4, thomas_chains=16, cluster=1, tl_levels=5, split_tile_rows=8192, split_threads=512)
for kp in ([7], [4, 3], [3, 4], [5, 2], [2, 5], [4, 4], [3, 3]):
    for ch in (0, 8, 4, 2, 1):
        plan = tds.Plan(n, m, "float32", device=0)
        try:
            plan.set_params(k_pass=kp, chunk_systems=ch, **base)
        except tds.TdsError as e:
            print(kp, ch, "rejected", e)
            continue
        ws = plan.workspace()
        us = timeit(lambda: tds.solve_batched(plan, ta, tb, tc, td, out=x, workspace=ws))
        print(f"k_pass={kp} chunk={ch}: {us:.1f} us  {n * m / us / 1e3:.1f} Geq/s", flush=True)
