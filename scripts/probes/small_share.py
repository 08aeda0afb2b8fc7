"""Config 3 at small per-rank shares (strong scaling): graph-replay time of a
few explicit plans vs the tuned one (diagnostic).

    python scripts/probes/small_share.py [m ...]
"""
import sys

import torch

sys.path.insert(0, ".")
import paper_conf_ipps_davidsonzo11_b200 as tds  # noqa: E402

n = 1 << 20
ms = [int(v) for v in sys.argv[1:]] or [2, 4]
W = dict(cr_levels=4, thomas_chains=1, tl_levels=5, cluster=1)
PLANS = {
    "k7 t512": dict(W, k_pass=[7], split_threads=512, split_tile_rows=8192),
    "k7 t256": dict(W, k_pass=[7], split_threads=256, split_tile_rows=4096),
    "k8 t512": dict(W, k_pass=[8], cr_levels=3, split_threads=512, split_tile_rows=8192),
    "k8 t256": dict(W, k_pass=[8], cr_levels=3, split_threads=256, split_tile_rows=4096),
    "k8 t256 c4": dict(W, k_pass=[8], split_threads=256, split_tile_rows=4096),
    "k7 t512 xg8": dict(W, k_pass=[7], split_threads=512, split_tile_rows=8192, x_group=8),
}


def graph_time(plan, args, reps=200):
    ws = plan.workspace()
    x = torch.empty_like(args[3])
    s = torch.cuda.Stream()
    s.wait_stream(torch.cuda.current_stream())
    with torch.cuda.stream(s):
        tds.solve_batched(plan, *args, out=x, workspace=ws)
    torch.cuda.current_stream().wait_stream(s)
    torch.cuda.synchronize()
    g = torch.cuda.CUDAGraph()
    with torch.cuda.graph(g):
        tds.solve_batched(plan, *args, out=x, workspace=ws)
    for _ in range(20):
        g.replay()
    torch.cuda.synchronize()
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    e0.record()
    for _ in range(reps):
        g.replay()
    e1.record()
    torch.cuda.synchronize()
    return e0.elapsed_time(e1) / reps


for m in ms:
    args = tds.generate(n, m, "float32", seed=3)
    tuned = tds.Plan(n, m, "float32", device=0)
    tuned.tune()
    print(f"m={m} tuned {tuned.info['k_pass']} t{tuned.info['split_threads']}: {graph_time(tuned, args) * 1e3:.1f} us",
          flush=True)
    for name, p in PLANS.items():
        plan = tds.Plan(n, m, "float32", device=0)
        try:
            plan.set_params(**p)
        except tds.TdsError as e:
            print(f"m={m} {name}: rejected {e}")
            continue
        print(f"m={m} {name}: {graph_time(plan, args) * 1e3:.1f} us", flush=True)
