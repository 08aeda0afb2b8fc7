"""Probe: host cost of one tds_solve_batched call vs its device time (config 3
tuned plan).  Diagnostic only."""
import json, os, sys, time
import torch
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_ipps_davidsonzo11_b200 as tds  # noqa: E402
from paper_conf_ipps_davidsonzo11_b200 import api  # noqa: E402
n, m = 1 << 20, 16
g = torch.Generator(device="cuda").manual_seed(1)
a, c, d = (torch.rand(m, n, device="cuda", generator=g) * 2 - 1 for _ in range(3))
b = a.abs() + c.abs() + 1
x = torch.empty_like(d)
plan = tds.Plan(n, m, "float32", mode="static")
plan.set_params(k_pass=[7], cr_levels=4, thomas_chains=16, tl_levels=5, split_threads=512, cluster=1)
ws = plan.workspace()
for _ in range(5):
    tds.solve_batched(plan, a, b, c, d, out=x, workspace=ws)
torch.cuda.synchronize()
N = 200
t0 = time.perf_counter()
for _ in range(N):
    tds.solve_batched(plan, a, b, c, d, out=x, workspace=ws)
t1 = time.perf_counter()
torch.cuda.synchronize()
t2 = time.perf_counter()
print(json.dumps({"host_us_per_call": (t1 - t0) / N * 1e6, "wall_us_per_call_incl_sync": (t2 - t0) / N * 1e6}))
for stage in range(3):
    t0 = time.perf_counter()
    for _ in range(N):
        api.solve_stages(plan, a, b, c, d, x, ws, stage, stage)
    t1 = time.perf_counter()
    torch.cuda.synchronize()
    print(json.dumps({"stage": stage, "host_us_per_call": (t1 - t0) / N * 1e6}))
# raw ctypes call cost
lib = plan._lib
t0 = time.perf_counter()
for _ in range(N):
    lib.tds_version()
t1 = time.perf_counter()
print(json.dumps({"ctypes_noop_us": (t1 - t0) / N * 1e6}))
