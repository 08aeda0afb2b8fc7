"""The paper's strided base-kernel variant vs the de-interleaved path (same k,
same on-chip form) and the tuned plan, per-kernel times (diagnostic)."""
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


for name, n, m, ks in [("cfg2 256 x 65536", 65536, 256, (3,)), ("cfg4 4096 x 16384", 16384, 4096, (1,)),
                       ("2048 x 32768", 32768, 2048, (2,))]:
    a, b, c, d = (torch.from_numpy(v).cuda() for v in inputs.generate(n, m, np.float32, seed=1))
    x = torch.empty_like(d)
    for k in ks:
        for sv in (0, 1):
            plan = tds.Plan(n, m, "float32", device=0)
            plan.set_params(k_pass=[k], cr_levels=4, thomas_chains=1, cluster=1, tl_levels=5, strided=sv)
            ws = plan.workspace()
            us = timeit(lambda: tds.solve_batched(plan, a, b, c, d, out=x, workspace=ws))
            print(f"{name} k={k} strided={sv}: {us:.1f} us ({n * m / us / 1e3:.1f} Geq/s)", flush=True)
    plan = tds.Plan(n, m, "float32", device=0)
    plan.tune()
    ws = plan.workspace()
    us = timeit(lambda: tds.solve_batched(plan, a, b, c, d, out=x, workspace=ws))
    print(f"{name} tuned ({plan.info['k_pass']}, cluster {plan.info['cluster']}, strided {plan.info['strided']}): "
          f"{us:.1f} us", flush=True)
