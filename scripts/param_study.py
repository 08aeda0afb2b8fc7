#!/usr/bin/env python
"""The paper's parameter-selection study re-run on B200.

PAPER.md §IV-E / Fig. 7 compares untuned (DEFAULT), statically
tuned (STATIC) and self-tuned (TUNED) parameters on 1Kx1K, 2Kx2K, 4Kx4K and
1x2M systems; Fig. 5 sweeps the stage-2->3 switch (subsystem
size, i.e. k) and Fig. 6 the stage-3->4 switch (Thomas chains T).
This script times all three modes on Fig. 7's workloads (fp32, as the paper's
figures; R12) plus both sweeps on 16 x 2^20, and writes one JSON line per
measurement plus a markdown table.

    python scripts/param_study.py --out gpurun_out/param_study
"""
import argparse
import json
import os
import sys
import tempfile

import numpy as np

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))

FIG7 = [("1Kx1K", 1024, 1024), ("2Kx2K", 2048, 2048), ("4Kx4K", 4096, 4096), ("1x2M", 1 << 21, 1)]


def time_plan(tds, plan, ta, tb, tc, td, x, reps):
    import torch
    ws = plan.workspace()
    for _ in range(3):
        tds.solve_batched(plan, ta, tb, tc, td, out=x, workspace=ws)
    torch.cuda.synchronize()
    ms = []
    for _ in range(reps):
        e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        e0.record()
        tds.solve_batched(plan, ta, tb, tc, td, out=x, workspace=ws)
        e1.record()
        torch.cuda.synchronize()
        ms.append(e0.elapsed_time(e1))
    return float(np.median(ms)), float(np.min(ms))


def plan_summary(info):
    return {k: info[k] for k in ("k", "k_pass", "n_sub", "cr_levels", "thomas_chains", "cluster", "tl_levels",
                                 "split_threads")}


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--out", default="gpurun_out/param_study")
    ap.add_argument("--reps", type=int, default=30)
    args = ap.parse_args()
    import torch
    import oracle
    import paper_conf_ipps_davidsonzo11_b200 as tds
    from paper_conf_ipps_davidsonzo11_b200 import inputs

    os.makedirs(os.path.dirname(args.out) or ".", exist_ok=True)
    lines = []

    def emit(rec):
        lines.append(rec)
        print(json.dumps(rec), flush=True)

    # ---- Fig. 7: DEFAULT vs STATIC vs TUNED
    for name, n, m in FIG7:
        a, b, c, d = inputs.generate(n, m, np.float32, seed=7)
        ta, tb, tc, td = (torch.from_numpy(v).cuda() for v in (a, b, c, d))
        x = torch.empty_like(td)
        for mode in ("default", "static", "tuned"):
            plan = tds.Plan(n, m, "float32", device=0, mode="static" if mode == "tuned" else mode)
            trials = 0
            if mode == "tuned":
                cache = tempfile.mktemp(suffix=".tds_tune")
                trials = plan.tune(cache_path=cache)
                if os.path.exists(cache):
                    os.unlink(cache)
            med, mn = time_plan(tds, plan, ta, tb, tc, td, x, args.reps)
            xs = x[: min(m, 4)].cpu().numpy()
            err = oracle.rel_err(xs, oracle.thomas(a[: min(m, 4)], b[: min(m, 4)], c[: min(m, 4)], d[: min(m, 4)]))
            emit({"study": "fig7", "workload": name, "n": n, "m": m, "mode": mode, "ms_median": med, "ms_min": mn,
                  "eq_per_s": n * m / (med / 1e3), "tune_trials": trials, "rel_err_sample": err,
                  "plan": plan_summary(plan.info)})
        del ta, tb, tc, td, x

    # ---- Fig. 5 / Fig. 6 sweeps on 16 x 2^20 (on-chip c = 4, warp form)
    n, m = 1 << 20, 16
    a, b, c, d = inputs.generate(n, m, np.float32, seed=3)
    ta, tb, tc, td = (torch.from_numpy(v).cuda() for v in (a, b, c, d))
    x = torch.empty_like(td)
    for k in range(5, 10):  # stage 2->3: subsystem size 2^20 / 2^k
        plan = tds.Plan(n, m, "float32", device=0)
        try:
            kp = [k] if k <= 8 else [k - k // 2, k // 2]
            c_lv = 4 if (n >> k) >= 8192 else 3
            plan.set_params(k_pass=kp, cr_levels=c_lv, thomas_chains=8, tl_levels=5, cluster=1)
        except tds.TdsError as e:
            emit({"study": "fig5", "k": k, "error": str(e)})
            continue
        med, mn = time_plan(tds, plan, ta, tb, tc, td, x, args.reps)
        emit({"study": "fig5", "k": k, "n_sub": n >> k, "ms_median": med, "ms_min": mn,
              "eq_per_s": n * m / (med / 1e3), "plan": plan_summary(plan.info)})
    for T in (1, 2, 4, 8, 16):  # stage 3->4: Thomas chains on the per-warp system (tl_levels = 5)
        plan = tds.Plan(n, m, "float32", device=0)
        plan.set_params(k_pass=[7], cr_levels=4, thomas_chains=T, tl_levels=5, cluster=1)
        med, mn = time_plan(tds, plan, ta, tb, tc, td, x, args.reps)
        emit({"study": "fig6_warp", "T": T, "ms_median": med, "eq_per_s": n * m / (med / 1e3),
              "plan": plan_summary(plan.info)})
    for T in (1, 4, 16, 64, 256):  # the paper's form: CR in registers, then PCR-Thomas in shared memory
        plan = tds.Plan(n, m, "float32", device=0)
        try:
            plan.set_params(k_pass=[7], cr_levels=4, thomas_chains=T, tl_levels=0, cluster=1)
        except tds.TdsError as e:
            emit({"study": "fig6_smem", "T": T, "error": str(e)})
            continue
        med, mn = time_plan(tds, plan, ta, tb, tc, td, x, args.reps)
        emit({"study": "fig6_smem", "T": T, "ms_median": med, "eq_per_s": n * m / (med / 1e3),
              "plan": plan_summary(plan.info)})

    del ta, tb, tc, td, x
    # ---- the paper's load variants (tuned per workload P:L713-721) on Fig. 7's
    # 2Kx2K and 4Kx4K workloads at one-pass k = 3 / 4: de-interleaved (strided 0, warp form),
    # strided gather (1), coalesced groups with global fallback (2) over a Fig. 6 T sweep
    for name, n, m in FIG7[1:3]:
        a, b, c, d = inputs.generate(n, m, np.float32, seed=4)
        ta, tb, tc, td = (torch.from_numpy(v).cuda() for v in (a, b, c, d))
        x = torch.empty_like(td)
        for k in (3, 4):
            runs = [(0, dict(cr_levels=4, thomas_chains=1, tl_levels=5)), (1, dict(cr_levels=4, thomas_chains=1,
                                                                                    tl_levels=5))]
            runs += [(2, dict(cr_levels=0, thomas_chains=T, tl_levels=0)) for T in (1, 4, 16, 64)]
            for sv, kw in runs:
                plan = tds.Plan(n, m, "float32", device=0)
                try:
                    plan.set_params(k_pass=[k], cluster=1, strided=sv, **kw)
                except tds.TdsError as e:
                    emit({"study": "load_variants", "workload": name, "k": k, "strided": sv, "error": str(e)})
                    continue
                med, mn = time_plan(tds, plan, ta, tb, tc, td, x, args.reps)
                emit({"study": "load_variants", "workload": name, "k": k, "strided": sv, "T": kw["thomas_chains"],
                      "n_sub": -(-n >> k), "ms_median": med, "eq_per_s": n * m / (med / 1e3),
                      "plan": plan_summary(plan.info)})
        del ta, tb, tc, td, x

    with open(args.out + ".jsonl", "w") as f:
        for r in lines:
            f.write(json.dumps(r) + "\n")
    md = ["| workload | DEFAULT ms | STATIC ms | TUNED ms | TUNED plan | static / default | tuned / default |",
          "|---|---|---|---|---|---|---|"]
    for name, _, _ in FIG7:
        r = {x["mode"]: x for x in lines if x.get("study") == "fig7" and x["workload"] == name}
        p = r["tuned"]["plan"]
        md.append(f"| {name} | {r['default']['ms_median']:.4f} | {r['static']['ms_median']:.4f} | "
                  f"{r['tuned']['ms_median']:.4f} | k={p['k']} {p['k_pass']} c={p['cr_levels']} T={p['thomas_chains']} "
                  f"C={p['cluster']} tl={p['tl_levels']} | {r['static']['ms_median'] / r['default']['ms_median']:.2f} | "
                  f"{r['tuned']['ms_median'] / r['default']['ms_median']:.2f} |")
    md += ["", "| Fig. 5: k | n_sub | ms | eq/s |", "|---|---|---|---|"]
    for r in lines:
        if r.get("study") == "fig5" and "ms_median" in r:
            md.append(f"| {r['k']} | {r['n_sub']} | {r['ms_median']:.4f} | {r['eq_per_s']:.3g} |")
    md += ["", "| Fig. 6: form | T | ms | eq/s |", "|---|---|---|---|"]
    for r in lines:
        if r.get("study", "").startswith("fig6") and "ms_median" in r:
            md.append(f"| {r['study'][5:]} | {r['T']} | {r['ms_median']:.4f} | {r['eq_per_s']:.3g} |")
    md += ["", "| load variant (P:L279-295) | workload | k | n_sub | T | ms | eq/s |", "|---|---|---|---|---|---|---|"]
    names = {0: "de-interleaved (B200 primary, warp form)", 1: "strided gather", 2: "coalesced + global fallback"}
    for r in lines:
        if r.get("study") == "load_variants" and "ms_median" in r:
            md.append(f"| {names[r['strided']]} | {r['workload']} | {r['k']} | {r['n_sub']} | {r['T']} | "
                      f"{r['ms_median']:.4f} | {r['eq_per_s']:.3g} |")
    with open(args.out + ".md", "w") as f:
        f.write("\n".join(md) + "\n")


if __name__ == "__main__":
    main()
