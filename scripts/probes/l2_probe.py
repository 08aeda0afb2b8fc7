"""Probe: per-kernel time per equation of the config-3 tuned plan as the batch
shrinks into L2 (m = 1..16 systems of 2^20 rows), and chunked runs at m = 16.
Prints one JSON line per case.  Diagnostic only (not part of the product)."""
import json
import os
import sys

import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.dirname(os.path.abspath(__file__)))))
import paper_conf_ipps_davidsonzo11_b200 as tds  # noqa: E402
from paper_conf_ipps_davidsonzo11_b200 import api  # noqa: E402

n = 1 << 20
TUNED = dict(k_pass=[7], cr_levels=4, thomas_chains=16, tl_levels=5, split_threads=512, cluster=1)


def make(m):
    g = torch.Generator(device="cuda").manual_seed(1)
    a = torch.rand(m, n, device="cuda", generator=g) * 2 - 1
    c = torch.rand(m, n, device="cuda", generator=g) * 2 - 1
    d = torch.rand(m, n, device="cuda", generator=g) * 2 - 1
    b = a.abs() + c.abs() + 1
    return a, b, c, d


def time_stage(plan, args, x, ws, first, last, reps=30):
    s = torch.cuda.current_stream()
    for _ in range(3):
        api.solve_stages(plan, *args, x, ws, first, last)
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    ts = []
    for _ in range(reps):
        e0.record(s)
        api.solve_stages(plan, *args, x, ws, first, last)
        e1.record(s)
        e1.synchronize()
        ts.append(e0.elapsed_time(e1))
    ts.sort()
    return ts[len(ts) // 2]


for m in (1, 2, 4, 8, 16):
    args = make(m)
    x = torch.empty_like(args[3])
    plan = tds.Plan(n, m, "float32", mode="static")
    plan.set_params(**TUNED)
    ws = plan.workspace()
    nl = plan.info["launches"] if "launches" in plan.info else 3
    res = {"m": m}
    names = ["split", "onchip", "place"]
    for i in range(3):
        res[names[i] + "_ns_per_meq"] = time_stage(plan, args, x, ws, i, i) * 1e6 / (m * n / 1e6) / 1e3
    res["all_ns_per_meq"] = time_stage(plan, args, x, ws, 0, 2) * 1e6 / (m * n / 1e6) / 1e3
    print(json.dumps(res), flush=True)

m = 16
args = make(m)
x = torch.empty_like(args[3])
for cs in (1, 2, 4, 8):
    plan = tds.Plan(n, m, "float32", mode="static")
    plan.set_params(chunk_systems=cs, **TUNED)
    ws = plan.workspace()
    nl = (m // cs) * 3
    t = time_stage(plan, args, x, ws, 0, nl - 1)
    print(json.dumps({"m": m, "chunk_systems": cs, "ms": t, "ns_per_meq": t * 1e3 / (m * n / 1e6)}), flush=True)
