"""Probe: host cost of one tds_solve_batched call vs its device time (config 3
tuned plan).  Diagnostic only."""
import json, os, sys, time
import torch
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.dirname(os.path.abspath(__file__)))))
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
# the C ABI alone (no Python argument checks): raw pointers through ctypes
import ctypes  # noqa: E402
h = plan.handle
ptrs = [ctypes.c_void_p(t.data_ptr()) for t in (a, b, c, d, x)]
wsp, wsb = ctypes.c_void_p(ws.data_ptr()), ctypes.c_size_t(ws.numel())
stp = ctypes.c_void_p(torch.cuda.current_stream().cuda_stream)
for _ in range(5):
    lib.tds_solve_batched(h, *ptrs, wsp, wsb, stp)
torch.cuda.synchronize()
t0 = time.perf_counter()
for _ in range(N):
    lib.tds_solve_batched(h, *ptrs, wsp, wsb, stp)
t1 = time.perf_counter()
torch.cuda.synchronize()
print(json.dumps({"c_abi_host_us_per_call": (t1 - t0) / N * 1e6}))
# config 1 (k = 0, one system of 1024): host cost and device time per call
n1 = 1024
a1, c1, d1 = (torch.rand(1, n1, device="cuda") * 2 - 1 for _ in range(3))
b1 = a1.abs() + c1.abs() + 1
x1 = torch.empty_like(d1)
p1 = tds.Plan(n1, 1, "float32", mode="static")
p1s = [ctypes.c_void_p(t.data_ptr()) for t in (a1, b1, c1, d1, x1)]
for _ in range(5):
    lib.tds_solve_batched(p1.handle, *p1s, None, ctypes.c_size_t(0), stp)
torch.cuda.synchronize()
t0 = time.perf_counter()
for _ in range(N):
    lib.tds_solve_batched(p1.handle, *p1s, None, ctypes.c_size_t(0), stp)
t1 = time.perf_counter()
torch.cuda.synchronize()
t2 = time.perf_counter()
print(json.dumps({"cfg1_c_abi_host_us_per_call": (t1 - t0) / N * 1e6, "cfg1_wall_us_per_call": (t2 - t0) / N * 1e6}))
