#!/usr/bin/env python
"""The tuner's choices evidenced by ncu counters (north_star):
for each BASELINE shape, the tuned plan next to the alternatives the climb
rejected, timed by CUDA events (mode "time") and profiled per kernel under
    ncu --metrics <METRICS> --csv --log-file L python scripts/tuner_ncu.py ncu
(mode "ncu": one solve per plan, launches in plan order; the "plan" lines on
stdout give each plan's launch count so the CSV rows can be attributed).
    python scripts/tuner_ncu.py report L time.txt > profiles/<tag>_tuner_ncu.md
"""
import csv
import json
import sys

METRICS = ("gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum,"
           "sm__warps_active.avg.pct_of_peak_sustained_active,smsp__issue_active.avg.pct_of_peak_sustained_active,"
           "l1tex__data_bank_conflicts_pipe_lsu_mem_shared_op_st.sum,"
           "l1tex__data_bank_conflicts_pipe_lsu_mem_shared_op_ld.sum,launch__grid_size,launch__block_size")

W5 = dict(tl_levels=5, thomas_chains=1, cluster=1)
CACHE = "/tmp/tds_tuner_ncu.tune"
MODE = [""]
SHAPES = {
    "config 2 (256 x 65536)": (65536, 256, [
        ("k=0, 8-CTA clusters", dict(k_pass=[], cr_levels=4, **dict(W5, cluster=8))),
        ("k=0, 16-CTA cluster (generic)", dict(k_pass=[], cr_levels=3, thomas_chains=32, tl_levels=4, cluster=16)),
        ("k=3 split + pipe (STATIC k)", dict(k_pass=[3], cr_levels=4, **W5)),
        ("k=4 split + pipe", dict(k_pass=[4], cr_levels=4, **W5))]),
    "config 3 (16 x 2^20)": (1 << 20, 16, [
        ("k=7 one pass + pipe", dict(k_pass=[7], cr_levels=4, **W5)),
        ("k=8 one pass + pipe", dict(k_pass=[8], cr_levels=4, **W5)),
        ("k=4 + 8-CTA cluster (generic)", dict(k_pass=[4], cr_levels=3, thomas_chains=32, tl_levels=3, cluster=8)),
        ("k=7 + smem PCR-Thomas T=64", dict(k_pass=[7], cr_levels=4, thomas_chains=64, tl_levels=0, cluster=1)),
        ("k=7 in two passes (4+3)", dict(k_pass=[4, 3], cr_levels=4, **W5))]),
    "config 4 (4096 x 16384)": (16384, 4096, [
        ("k=0, 2-CTA clusters", dict(k_pass=[], cr_levels=4, **dict(W5, cluster=2))),
        ("k=1 split + pipe (STATIC k)", dict(k_pass=[1], cr_levels=4, **W5)),
        ("k=0, 4-CTA clusters", dict(k_pass=[], cr_levels=4, **dict(W5, cluster=4)))]),
}


def plans(tds):
    for shape, (n, m, alts) in SHAPES.items():
        tuned = tds.Plan(n, m, "float32", device=0)
        # mode "time" tunes and caches; mode "ncu" must hit the cache (no trial kernels in the launch list)
        trials = tuned.tune(cache_path=CACHE)
        assert MODE[0] == "time" or trials == 0, "run mode 'time' first (tune cache)"
        yield shape, n, m, "TUNED " + str(tuned.params_list()), tuned
        for label, p in alts:
            q = tds.Plan(n, m, "float32", device=0)
            try:
                q.set_params(**p)
            except tds.TdsError as e:
                print(json.dumps({"shape": shape, "plan": label, "error": str(e)}), flush=True)
                continue
            yield shape, n, m, label, q


def run(mode):
    MODE[0] = mode
    import torch
    sys.path.insert(0, ".")
    import paper_conf_ipps_davidsonzo11_b200 as tds
    cache = {}
    for shape, n, m, label, plan in plans(tds):
        if (n, m) not in cache:
            cache.clear()
            a, b, c, d = tds.generate(n, m, "float32", seed=3)
            cache[(n, m)] = (a, b, c, d, torch.empty_like(d))
        a, b, c, d, x = cache[(n, m)]
        ws = plan.workspace()
        rec = {"shape": shape, "plan": label, "launches": plan.info["launches"]}
        if mode == "time":
            for _ in range(3):
                tds.solve_batched(plan, a, b, c, d, out=x, workspace=ws)
            torch.cuda.synchronize()
            ts = []
            for _ in range(20):
                e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
                e0.record()
                tds.solve_batched(plan, a, b, c, d, out=x, workspace=ws)
                e1.record()
                torch.cuda.synchronize()
                ts.append(e0.elapsed_time(e1))
            rec["ms_median"] = sorted(ts)[len(ts) // 2]
        else:
            torch.cuda.synchronize()
            tds.solve_batched(plan, a, b, c, d, out=x, workspace=ws)
            torch.cuda.synchronize()
        print(json.dumps(rec), flush=True)


def report(csv_path, time_path, ncu_stdout):
    times = {}
    for l in open(time_path):
        if l.startswith("{"):
            r = json.loads(l)
            times[(r["shape"], r["plan"])] = r.get("ms_median")
    order = [json.loads(l) for l in open(ncu_stdout) if l.startswith("{") and "launches" in l]
    rows = list(csv.reader(open(csv_path)))
    hi = [i for i, r in enumerate(rows) if r and r[0] == "ID"][0]
    h = rows[hi]
    per = {}
    for r in rows[hi + 1:]:
        d = dict(zip(h, r))
        per.setdefault(d["ID"], {"kernel": d["Kernel Name"].split("(")[0].replace("void ", "")})[d["Metric Name"]] = \
            d["Metric Value"]
    launches = [per[k] for k in sorted(per, key=int) if "generate" not in per[k]["kernel"]]
    print("# The tuner's choices against rejected alternatives, with ncu counters\n")
    print("`scripts/tuner_ncu.py`: CUDA-event median per solve (20 runs, warm) and, per kernel, one ncu replay "
          "(cold L2, serialised): duration, DRAM bytes, warps active, issue active, shared-memory bank conflicts. "
          "The TUNED row is what `tds_tune` chose (its integer parameter list); the others are the STATIC k or "
          "neighbours the hill climb tried.\n")
    i = 0
    cur = None
    for o in order:
        if o["shape"] != cur:
            cur = o["shape"]
            print(f"\n## {cur}\n")
            print("| plan | solve ms | kernel | ncu us | DRAM MB r / w | warps active % | issue active % | "
                  "smem conflicts st / ld |")
            print("|---|---|---|---|---|---|---|---|")
        t = times.get((o["shape"], o["plan"]))
        for j in range(o["launches"]):
            k = launches[i]
            i += 1
            f = lambda key: float(k.get(key, "0").replace(",", "") or 0)
            print(f"| {o['plan'] if j == 0 else ''} | {'' if j else (f'{t:.4f}' if t else '')} | {k['kernel'][:42]} | "
                  f"{f('gpu__time_duration.sum') / 1e3:.1f} | "
                  f"{f('dram__bytes_read.sum') / 1e6:.0f} / {f('dram__bytes_write.sum') / 1e6:.0f} | "
                  f"{f('sm__warps_active.avg.pct_of_peak_sustained_active'):.0f} | "
                  f"{f('smsp__issue_active.avg.pct_of_peak_sustained_active'):.0f} | "
                  f"{f('l1tex__data_bank_conflicts_pipe_lsu_mem_shared_op_st.sum'):.0f} / "
                  f"{f('l1tex__data_bank_conflicts_pipe_lsu_mem_shared_op_ld.sum'):.0f} |")


if __name__ == "__main__":
    if sys.argv[1] == "report":
        report(sys.argv[2], sys.argv[3], sys.argv[4])
    elif sys.argv[1] == "metrics":
        print(METRICS)
    else:
        run(sys.argv[1])
