#!/usr/bin/env python
"""Attribute ncu per-SASS warp-stall samples to CUDA source lines.

    python scripts/ncu_lines.py gpurun_out/prof.ncu-rep [mangled-substring] [top] [ncu-kernel-regex]

ncu's SASS page gives samples per instruction address; the cubin's line table
(nvdisasm -g over the cubin extracted from libtds.so) maps each address to a
source line.  Addresses are matched by offset from the function start.
"""
import collections
import csv
import io
import os
import re
import subprocess
import sys
import tempfile

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
LIB = os.path.join(ROOT, "paper_conf_ipps_davidsonzo11_b200", "libtds.so")


def sass_samples(rep, kfilter=""):
    cmd = ["ncu", "-i", rep, "--page", "source", "--csv", "--print-source", "sass"]
    if kfilter:
        cmd += ["-k", "regex:" + kfilter]
    out = subprocess.run(cmd, capture_output=True, text=True).stdout
    rows = list(csv.reader(io.StringIO(out)))
    name = rows[0][1] if rows and rows[0][0] == "Kernel Name" else ""
    hi = [i for i, r in enumerate(rows) if r and r[0] == "Address"][0]
    h = rows[hi]
    si = h.index("Warp Stall Sampling (All Samples)")
    body = []
    for r in rows[hi + 1:]:
        if r and r[0] == "Kernel Name":
            break
        if len(r) > si and r[si].isdigit():
            body.append(r)
    base = int(body[0][0], 16)
    stall_cols = [(i, c[len("stall_"):]) for i, c in enumerate(h) if c.startswith("stall_") and "Not Issued" not in c]
    out = []
    for r in body:
        st = {nm: int(r[i]) for i, nm in stall_cols if i < len(r) and r[i].isdigit() and int(r[i]) > 0}
        out.append((int(r[0], 16) - base, int(r[si]), r[h.index("Source")].strip(), st))
    return name, out


def line_table(mangled_substr):
    tmp = tempfile.mkdtemp()
    subprocess.run(["cuobjdump", "-xelf", "all", LIB], cwd=tmp, capture_output=True)
    table = {}
    for f in os.listdir(tmp):
        txt = subprocess.run(["nvdisasm", "-g", "-c", os.path.join(tmp, f)], capture_output=True, text=True).stdout
        cur, line, inside = None, None, False
        for l in txt.splitlines():
            m = re.match(r"\s*\.text\.(\S+):", l)
            if m:
                inside = mangled_substr in m.group(1)
                cur = m.group(1)
                continue
            if not inside:
                continue
            m = re.search(r"//## File \"([^\"]+)\", line (\d+)", l)
            if m:
                line = f"{os.path.basename(m.group(1))}:{m.group(2)}"
                continue
            m = re.match(r"\s*/\*([0-9a-f]{4,})\*/", l)
            if m and line:
                table[(cur, int(m.group(1), 16))] = line
    return table


def main():
    rep = sys.argv[1]
    sub = sys.argv[2] if len(sys.argv) > 2 else ""
    top = int(sys.argv[3]) if len(sys.argv) > 3 else 30
    name, samples = sass_samples(rep, sys.argv[4] if len(sys.argv) > 4 else "")
    # pick the mangled function whose instruction count best matches
    table = line_table(sub)
    funcs = collections.defaultdict(dict)
    for (fn, off), ln in table.items():
        funcs[fn][off] = ln
    best = max(funcs, key=lambda fn: sum(1 for off, _, _, _ in samples if off in funcs[fn])) if funcs else None
    agg = collections.Counter()
    why = collections.defaultdict(collections.Counter)
    tot = sum(s for _, s, _, _ in samples) or 1
    for off, s, _, st in samples:
        ln = funcs[best].get(off, "?") if best else "?"
        agg[ln] += s
        why[ln].update(st)
    print(f"{name[:90]}  ({best})")
    for ln, s in agg.most_common(top):
        w = ", ".join(f"{k} {v * 100 // max(s, 1)}%" for k, v in why[ln].most_common(3))
        print(f"  {s / tot * 100:5.1f}%  {ln:28s} {w}")


if __name__ == "__main__":
    main()
