"""One shape, one load variant (for ncu --set full of the coalesced kernel)."""
import sys

import numpy as np
import torch

sys.path.insert(0, ".")
import paper_conf_ipps_davidsonzo11_b200 as tds  # noqa: E402
from paper_conf_ipps_davidsonzo11_b200 import inputs  # noqa: E402

n, m, k, T = (int(v) for v in sys.argv[1:5])
a, b, c, d = (torch.from_numpy(v).cuda() for v in inputs.generate(n, m, np.float32, seed=1))
x = torch.empty_like(d)
plan = tds.Plan(n, m, "float32", device=0)
plan.set_params(k_pass=[k], cr_levels=0, thomas_chains=T, cluster=1, tl_levels=0, strided=2)
ws = plan.workspace()
for _ in range(2):
    tds.solve_batched(plan, a, b, c, d, out=x, workspace=ws)
torch.cuda.synchronize()
