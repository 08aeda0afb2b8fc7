#!/usr/bin/env python
"""Publish one gpu_final.sh run into profiles/: bench lines of every config,
per-launch lists (duration + DRAM bytes) of every config, ncu --set full
summaries of the config-3 kernels, and profiles/ncu_traffic.json (the
per-launch DRAM traffic bench.py reports as roofline.traffic).

    python scripts/publish_final.py <tag>
"""
import collections
import csv
import json
import os
import statistics
import subprocess
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
G = os.path.join(ROOT, "gpurun_out")
P = os.path.join(ROOT, "profiles")
CFGS = ["cfg3_f32", "cfg3_f64", "cfg2_f32", "cfg4_f32", "cfg1_f32", "cfg5_f32"]


def stage_of(kernel: str):
    k = kernel.split("(")[0].split("<")[0].replace("void ", "").replace("tds::", "").strip()
    if k.startswith("split_"):
        return "split_pass"
    if k.startswith("onchip"):
        return "onchip_cr_pcr_thomas"
    if k.startswith("place_x"):
        return "place_x"
    return None


def launches(path):
    rows = list(csv.reader(open(path)))
    i = [k for k, r in enumerate(rows) if r and r[0] == "ID"][0]
    h = rows[i]
    by = collections.OrderedDict()
    for r in rows[i + 1:]:
        if len(r) < len(h):
            continue
        lid = int(r[h.index("ID")])
        e = by.setdefault(lid, {"kernel": r[h.index("Kernel Name")], "grid": r[h.index("Grid Size")],
                                "block": r[h.index("Block Size")]})
        e[r[h.index("Metric Name")]] = float(r[h.index("Metric Value")].replace(",", ""))
    return list(by.values())


def main():
    tag = sys.argv[1]
    traffic = {}
    for cfg in CFGS:
        src = os.path.join(G, f"{tag}_launches_{cfg}.csv")
        if not os.path.exists(src):
            continue
        ls = launches(src)
        # stage keys in launch order within a step: split_pass_0, split_pass_1, ..., onchip, place_x
        per = collections.defaultdict(list)
        out = ["kernel,grid,block,gpu__time_duration.sum_ns,dram__bytes_read.sum,dram__bytes_write.sum"]
        p = 0
        for e in ls:
            st = stage_of(e["kernel"])
            if st is None:
                continue
            if st == "split_pass":
                key = f"split_pass_{p}"
                p += 1
            else:
                key = st
            if st == "onchip_cr_pcr_thomas":
                p = 0  # the next step's split passes count from 0 again
            per[key].append(e.get("dram__bytes_read.sum", 0) + e.get("dram__bytes_write.sum", 0))
            out.append(f'"{e["kernel"]}",{e["grid"].replace(", ", "x")},{e["block"].replace(", ", "x")},'
                       f'{e.get("gpu__time_duration.sum", 0):.0f},{e.get("dram__bytes_read.sum", 0):.0f},'
                       f'{e.get("dram__bytes_write.sum", 0):.0f}')
        traffic["config" + cfg[3:]] = {k: statistics.median(v) for k, v in per.items()}
        n, d = cfg[3:].split("_")
        open(os.path.join(P, f"{tag}_launches_{cfg}.txt"), "w").write(
            f"# ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none:"
            f" python bench.py --config {n} --dtype {d} --tune-cache <cached tuned plan> --steps 2 --warmup 1"
            f" --soak-s 0 --no-e2e --no-cpu-baseline (cold cache, serialised launches)\n" + "\n".join(out) + "\n")
        b = os.path.join(G, f"{tag}_bench_{cfg}.json")
        if os.path.exists(b):
            open(os.path.join(P, f"{tag}_bench_{cfg}.json"), "w").write(open(b).read())
    b = os.path.join(G, f"{tag}_bench_ref.json")
    if os.path.exists(b):
        open(os.path.join(P, f"{tag}_bench_ref.json"), "w").write(open(b).read())
    md = [f"# {tag}: ncu --set full summaries, config 3 fp32 (16 x 2^20), tuned plan", "",
          f"Command: `bash scripts/gpu_final.sh {tag}` (bench tunes and caches the plan; ncu runs read the cache). "
          "Captures: `ncu --set full --clock-control none --import-source on -k regex:<kernel> -s 2 -c 1` "
          "(cold L2, serialised).", "", "```"]
    for k in ("split_pipe", "onchip", "place_x", "split_pipe_f64", "cpipe_cfg4"):
        rep = os.path.join(G, f"prof_{k}_{tag}.ncu-rep")
        if k in ("split_pipe_f64", "cpipe_cfg4"):
            md.append("")
            md.append(f"# {'config 3 fp64' if k == 'split_pipe_f64' else 'config 4 fp32'}")
        if os.path.exists(rep):
            md.append(subprocess.run([sys.executable, os.path.join(ROOT, "scripts", "ncu_summary.py"), rep],
                                     capture_output=True, text=True).stdout.rstrip())
            md.append("")
    md.append("```")
    open(os.path.join(P, f"{tag}_ncu.md"), "w").write("\n".join(md) + "\n")
    traffic["note"] = (f"dram__bytes_read.sum + dram__bytes_write.sum per launch (bytes, median over the launches of "
                       f"each stage) from the ncu launch lists {tag}_launches_<config>.txt (cold cache, serialised). "
                       "Writes look low where a kernel's output is still dirty in L2 when it ends.")
    json.dump(traffic, open(os.path.join(P, "ncu_traffic.json"), "w"), indent=1)
    print(json.dumps(traffic, indent=1))


if __name__ == "__main__":
    main()
