"""Probe: split-stage time of config 3 (16 x 2^20 fp32) for split kernel
variants (threads per CTA, k_p).  Diagnostic only.
    python scripts/probes/split_probe.py [--only THREADS KP]   (one variant, e.g. under ncu)"""
import json
import os
import sys

import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.dirname(os.path.abspath(__file__)))))
import paper_conf_ipps_davidsonzo11_b200 as tds  # noqa: E402
from paper_conf_ipps_davidsonzo11_b200 import api  # noqa: E402

n, m = 1 << 20, 16
g = torch.Generator(device="cuda").manual_seed(1)
a, c, d = (torch.rand(m, n, device="cuda", generator=g) * 2 - 1 for _ in range(3))
b = a.abs() + c.abs() + 1
x = torch.empty_like(d)
variants = [(512, 7), (256, 7), (512, 6), (256, 6), (512, 5), (512, 4), (256, 4), (512, 8)]
if len(sys.argv) > 2 and sys.argv[1] == "--only":
    variants = [(int(sys.argv[2]), int(sys.argv[3]))]
for th, kp in variants:
    plan = tds.Plan(n, m, "float32", mode="static")
    plan.set_params(k_pass=[kp], cr_levels=4, thomas_chains=16, split_threads=th, split_tile_rows=th * 16,
                    cluster=max(1, 1 << max(0, 7 - kp)), tl_levels=5 if kp >= 7 else 3)
    ws = plan.workspace()
    s = torch.cuda.current_stream()
    for _ in range(3):
        api.solve_stages(plan, a, b, c, d, x, ws, 0, 0)
    ts = []
    for _ in range(20):
        e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        e0.record(s)
        api.solve_stages(plan, a, b, c, d, x, ws, 0, 0)
        e1.record(s)
        e1.synchronize()
        ts.append(e0.elapsed_time(e1))
    ts.sort()
    ms = ts[len(ts) // 2]
    print(json.dumps({"threads": th, "k_p": kp, "split_ms": ms, "gbs_28B": 28 * n * m / ms / 1e6}), flush=True)
