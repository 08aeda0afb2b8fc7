"""Per-kernel view of the load variants (run under ncu --metrics gpu__time_duration.sum)."""
import sys

import numpy as np
import torch

sys.path.insert(0, ".")
import paper_conf_ipps_davidsonzo11_b200 as tds  # noqa: E402
from paper_conf_ipps_davidsonzo11_b200 import inputs  # noqa: E402

for n, m, k, T in [(2048, 16384, 3, 16), (65536, 256, 4, 128)]:
    a, b, c, d = (torch.from_numpy(v).cuda() for v in inputs.generate(n, m, np.float32, seed=1))
    x = torch.empty_like(d)
    for sv in (0, 1, 2):
        plan = tds.Plan(n, m, "float32", device=0)
        if sv == 2:
            plan.set_params(k_pass=[k], cr_levels=0, thomas_chains=T, cluster=1, tl_levels=0, strided=2)
        else:
            plan.set_params(k_pass=[k], cr_levels=4, thomas_chains=1, cluster=1, tl_levels=5, strided=sv)
        ws = plan.workspace()
        for _ in range(2):
            tds.solve_batched(plan, a, b, c, d, out=x, workspace=ws)
        torch.cuda.synchronize()
