"""Probe: config 3 (16 x 2^20 fp32) on-chip stage time for the tuned plan and
on-chip variants (c = 3: 8 rows x 1024 threads; c = 4: 16 rows x 512).  Diagnostic."""
import json
import sys

import torch

sys.path.insert(0, ".")
import paper_conf_ipps_davidsonzo11_b200 as tds  # noqa: E402
from paper_conf_ipps_davidsonzo11_b200 import api  # noqa: E402

n, m = 1 << 20, 16
a, b, c, d = tds.generate(n, m, "float32", seed=3)
x = torch.empty_like(d)
base = tds.Plan(n, m, "float32", mode="static")
base.tune()
print("tuned", base.params_list(), flush=True)
variants = {"tuned": {}, "c3": {"cr_levels": 3}, "c3_tl4": {"cr_levels": 3, "tl_levels": 4}}
for name, kw in variants.items():
    plan = tds.Plan(n, m, "float32", mode="static")
    plan.set_params_list(base.params_list())
    try:
        if kw:
            plan.set_params(**kw)
    except tds.TdsError as e:
        print(name, "rejected:", e, flush=True)
        continue
    ws = plan.workspace()
    S = plan.info["launches"]
    for _ in range(5):
        tds.solve_batched(plan, a, b, c, d, out=x, workspace=ws)
    ev = [[torch.cuda.Event(enable_timing=True) for _ in range(S + 1)] for _ in range(20)]
    torch.cuda.synchronize()
    for i in range(20):
        for st in range(S):
            ev[i][st].record()
            api.solve_stages(plan, a, b, c, d, x, ws, st, st)
        ev[i][S].record()
    torch.cuda.synchronize()
    per = [sorted(ev[i][st].elapsed_time(ev[i][st + 1]) for i in range(20))[10] for st in range(S)]
    print(json.dumps({"variant": name, "params": plan.params_list(), "stage_ms": per,
                      "onchip_form": plan.info.get("onchip_form")}), flush=True)
