#!/usr/bin/env python
"""Copy one gpu_prof.sh run into profiles/: ncu summaries (markdown), the
launch list, per-launch DRAM traffic (profiles/ncu_traffic.json) and the bench line.

    python scripts/publish_profiles.py <tag> <plan description>
"""
import csv
import io
import json
import os
import subprocess
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
G = os.path.join(ROOT, "gpurun_out")
P = os.path.join(ROOT, "profiles")
KINDS = [("split_pipe", "split_pass_0"), ("onchip", "onchip_cr_pcr_thomas"), ("place_x", "place_x")]


def raw_metric(rep, names):
    out = subprocess.run(["ncu", "-i", rep, "--page", "raw", "--csv"], capture_output=True, text=True).stdout
    rows = list(csv.reader(io.StringIO(out)))
    h, v = rows[0], rows[2]
    return {n: float(v[h.index(n)].replace(",", "")) for n in names if n in h}


def main():
    tag, desc = sys.argv[1], " ".join(sys.argv[2:])
    md = [f"# {tag}: ncu summaries, config 3 fp32 (16 x 2^20), {desc}", "",
          f"Command: `bash scripts/gpu_prof.sh {tag} --config 3` (bench tunes and caches the plan; the ncu runs "
          "read the cache).  Captures: `ncu --set full --clock-control none --import-source on -k regex:<kernel> "
          "-s 2 -c 1` (cold L2, serialised).", "", "```"]
    traffic = {}
    for k, key in KINDS:
        rep = os.path.join(G, f"prof_{k}_{tag}.ncu-rep")
        if not os.path.exists(rep):
            continue
        md.append(subprocess.run([sys.executable, os.path.join(ROOT, "scripts", "ncu_summary.py"), rep],
                                 capture_output=True, text=True).stdout.rstrip())
        md.append("")
        m = raw_metric(rep, ["dram__bytes_read.sum", "dram__bytes_write.sum"])
        unit_scale = 1e6  # ncu reports Mbyte
        traffic[key] = (m.get("dram__bytes_read.sum", 0) + m.get("dram__bytes_write.sum", 0)) * unit_scale
    md.append("```")
    open(os.path.join(P, f"{tag}_ncu.md"), "w").write("\n".join(md) + "\n")
    lines = open(os.path.join(G, f"launches_{tag}.csv")).read().splitlines()
    i = [k for k, l in enumerate(lines) if l.startswith('"ID"')][0]
    rows = list(csv.reader(lines[i:]))
    h = rows[0]
    out = ["kernel,grid,block,gpu__time_duration.sum_ns"]
    for r in rows[1:]:
        if len(r) >= len(h):
            out.append(f'"{r[h.index("Kernel Name")]}",{r[h.index("Grid Size")].replace(", ", "x")},'
                       f'{r[h.index("Block Size")].replace(", ", "x")},{r[h.index("Metric Value")]}')
    open(os.path.join(P, f"{tag}_launches.txt"), "w").write(
        "# ncu --metrics gpu__time_duration.sum --clock-control none: python bench.py --config 3 --tune-cache "
        "<cached plan> --steps 2 --warmup 1 --soak-s 0 --no-e2e --no-cpu-baseline (cold-cache, serialised)\n"
        + "\n".join(out) + "\n")
    tj = {"config3_f32": traffic,
          "note": f"dram__bytes_read.sum + dram__bytes_write.sum per launch from one ncu --set full capture each "
                  f"({tag}_ncu.md), {desc}. Writes look low where a kernel's output is still dirty in L2 when it ends."}
    json.dump(tj, open(os.path.join(P, "ncu_traffic.json"), "w"), indent=1)
    for src, dst in ((f"bench_{tag}.json", f"{tag}_bench_cfg3_f32.json"),):
        if os.path.exists(os.path.join(G, src)):
            open(os.path.join(P, dst), "w").write(open(os.path.join(G, src)).read())
    print("published", tag, traffic)


if __name__ == "__main__":
    main()
