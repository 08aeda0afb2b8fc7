"""One config-3 plan with a given x_group, solved a few times (ncu target)."""
import sys

import numpy as np
import torch

sys.path.insert(0, ".")
import paper_conf_ipps_davidsonzo11_b200 as tds  # noqa: E402
from paper_conf_ipps_davidsonzo11_b200 import inputs  # noqa: E402

G = int(sys.argv[1]) if len(sys.argv) > 1 else 8
n, m = 1 << 20, 16
a, b, c, d = inputs.generate(n, m, np.float32, seed=3)
ta, tb, tc, td = (torch.from_numpy(v).cuda() for v in (a, b, c, d))
x = torch.empty_like(td)
plan = tds.Plan(n, m, "float32", device=0)
plan.set_params(k_pass=[7], cr_levels=4, thomas_chains=16, cluster=1, tl_levels=5, x_group=G)
ws = plan.workspace()
for _ in range(4):
    tds.solve_batched(plan, ta, tb, tc, td, out=x, workspace=ws)
torch.cuda.synchronize()
