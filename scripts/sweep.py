#!/usr/bin/env python
"""Parameter sweeps on the GPU (the paper's Fig. 5 / Fig. 6 switch-point
studies, re-run on B200): time every kernel of the solve
for explicit plan parameters and print one JSON line per point.

    python scripts/sweep.py --n 1048576 --m 16 --grid '{"k_pass": [[4], [5], [2,2]], "cluster": [8, 16]}'
"""
import argparse
import itertools
import json
import os
import sys

import numpy as np

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--n", type=int, default=1 << 20)
    ap.add_argument("--m", type=int, default=16)
    ap.add_argument("--dtype", default="float32")
    ap.add_argument("--grid", default="{}", help="JSON dict: param -> list of values (cartesian product)")
    ap.add_argument("--points", default=None, help="JSON list of param dicts (instead of --grid)")
    ap.add_argument("--reps", type=int, default=20)
    ap.add_argument("--mode", default="static")
    args = ap.parse_args()

    import torch
    import paper_conf_ipps_davidsonzo11_b200 as tds
    from paper_conf_ipps_davidsonzo11_b200 import inputs

    dt = np.float32 if args.dtype == "float32" else np.float64
    a, b, c, d = inputs.generate(args.n, args.m, dt, seed=3)
    ta, tb, tc, td = (torch.from_numpy(v).cuda() for v in (a, b, c, d))
    x = torch.empty_like(td)
    if args.points:
        points = json.loads(args.points)
    else:
        grid = json.loads(args.grid)
        keys = list(grid)
        points = [dict(zip(keys, vals)) for vals in itertools.product(*(grid[k] for k in keys))]
    s = np.dtype(dt).itemsize
    eqs = args.n * args.m
    for pt in points:
        plan = tds.Plan(args.n, args.m, args.dtype, device=0, mode=args.mode)
        try:
            if pt:
                plan.set_params(**pt)
        except tds.TdsError as e:
            print(json.dumps({"params": pt, "error": str(e)}), flush=True)
            continue
        info = plan.info
        ws = plan.workspace()
        NL = info["launches"]
        S = info["passes"] + 1 + (1 if info["k"] > 0 else 0)
        for _ in range(3):
            tds.solve_batched(plan, ta, tb, tc, td, out=x, workspace=ws)
        torch.cuda.synchronize()
        ev = [[torch.cuda.Event(enable_timing=True) for _ in range(NL + 1)] for _ in range(args.reps)]
        e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        for i in range(args.reps):
            for st in range(NL):
                ev[i][st].record()
                tds.api.solve_stages(plan, ta, tb, tc, td, x, ws, st, st)
            ev[i][NL].record()
        e0.record()
        for i in range(args.reps):
            tds.solve_batched(plan, ta, tb, tc, td, out=x, workspace=ws)
        e1.record()
        torch.cuda.synchronize()
        stage = [float(np.median([sum(ev[i][st].elapsed_time(ev[i][st + 1]) for st in range(kind, NL, S))
                                  for i in range(args.reps)])) for kind in range(S)]
        total = e0.elapsed_time(e1) / args.reps  # whole solve, back to back (no events between kernels)
        keep = {k: info[k] for k in ("k", "k_pass", "cr_levels", "thomas_chains", "cluster", "tl_levels",
                                     "chunk_systems", "chunks", "onchip_threads", "theta", "split_segments",
                                     "n_sub")}
        print(json.dumps({"params": pt, "plan": keep, "stage_ms": [round(v, 4) for v in stage],
                          "total_ms": round(total, 4), "geq_per_s": round(eqs / total / 1e6, 2)}), flush=True)


if __name__ == "__main__":
    main()
