#!/usr/bin/env python
"""Copy the rest of a final-evidence run (scripts/gpu_r02fin.sh TAG) into profiles/:
param study, cuSPARSE context (+ markdown table), GPU test log, sanitizer logs,
mutation summary and fuzz log.  Companion of publish_final.py (bench lines, ncu)."""
import json
import os
import shutil
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
T = sys.argv[1]
G = os.path.join(ROOT, "gpurun_out", T)
P = os.path.join(ROOT, "profiles")
for src, dst in [("param_study.md", f"{T}_param_study.md"), ("param_study.jsonl", f"{T}_param_study.jsonl"),
                 ("cusparse.jsonl", f"{T}_cusparse_context.jsonl"), ("gputests.txt", f"{T}_gpu_tests.txt"),
                 ("fuzz.txt", f"{T}_fuzz.txt")]:
    shutil.copy(os.path.join(G, src), os.path.join(P, dst))
with open(os.path.join(P, f"{T}_sanitizer.txt"), "w") as f:
    f.write(f"# {T} compute-sanitizer run (scripts/sanitize.py under memcheck / racecheck / synccheck)\n")
    for tool in ("memcheck", "racecheck", "synccheck"):
        f.write(f"\n## {tool}\n```\n" + open(os.path.join(G, f"san_{tool}.txt")).read() + "```\n")
with open(os.path.join(P, f"{T}_mutation.md"), "w") as f:
    f.write(f"# {T} mutation run: every TDS_MUTATE site against tests/test_coupling.py\n")
    for k in range(1, 8):
        p = os.path.join(G, "mutation", f"mut{k}.log")
        if not os.path.exists(p):
            continue
        lines = [l for l in open(p).read().splitlines() if l.startswith("FAILED") or " passed" in l or " failed" in l]
        f.write(f"\n## mutant {k}\n```\n" + "\n".join(lines[-30:]) + "\n```\n")
rows = [json.loads(l) for l in open(os.path.join(G, "cusparse.jsonl")) if l.startswith("{")]
md = [f"# {T}: cuSPARSE context comparison (SURVEY §8(f) item 4)", "",
      "`python scripts/cusparse_context.py` on one B200: the same generated systems and device buffers as bench.py; "
      "device time by CUDA events, median of 20 after 3 warm-ups (cuSPARSE's in-place right-hand-side copy timed "
      "separately and subtracted). A library point of reference, not the paper's comparison system and not a target.",
      "", "| config | solver | ms | eq/s | relative residual |", "|---|---|---|---|---|"]
for r in rows:
    md.append(f"| {r['config']} | {r['solver']} | {r['ms']:.4f} | {r['eq_per_s']:.3e} | {r['residual']:.1e} |")
ratios = []
for cfg in sorted({r["config"] for r in rows}):
    cs = [r for r in rows if r["config"] == cfg and r["solver"] == "cusparseSgtsv2StridedBatch"]
    tt = [r for r in rows if r["config"] == cfg and r["solver"] == "tds (tuned)"]
    if cs and tt:
        ratios.append(f"config {cfg}: {cs[0]['ms'] / tt[0]['ms']:.1f}x")
md += ["", "tds (tuned) vs cusparseSgtsv2StridedBatch: " + ", ".join(ratios)]
open(os.path.join(P, f"{T}_cusparse_context.md"), "w").write("\n".join(md) + "\n")
print("published", T, ratios)
