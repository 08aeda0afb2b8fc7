"""One small solve through every kernel family (compute-sanitizer target).

    compute-sanitizer --tool memcheck|racecheck|synccheck|initcheck python scripts/sanitize.py

Each case is checked against the fp64 Thomas oracle; sizes are small so the
instrumented run finishes in minutes but still span several tiles / items.
"""
import sys

import numpy as np
import torch

sys.path.insert(0, ".")
import oracle  # noqa: E402
import paper_conf_ipps_davidsonzo11_b200 as tds  # noqa: E402
from paper_conf_ipps_davidsonzo11_b200 import inputs  # noqa: E402

F32, F64 = np.float32, np.float64
CASES = [  # (label, dtype, n, m, params or None for the static plan)
    ("k0 static (onchip)", F32, 1000, 3, None),
    ("k0 cpipe C=1", F32, 8192, 4, dict(k_pass=[], cr_levels=4, thomas_chains=16, cluster=1, tl_levels=5)),
    ("k0 cpipe C=2", F32, 16000, 3, dict(k_pass=[], cr_levels=4, thomas_chains=16, cluster=2, tl_levels=5)),
    ("k0 cpipe C=8", F32, 65536, 2, dict(k_pass=[], cr_levels=4, thomas_chains=16, cluster=8, tl_levels=5)),
    ("k0 cluster onchip C=4", F32, 30000, 2, dict(k_pass=[], cr_levels=3, thomas_chains=32, cluster=4, tl_levels=2)),
    ("split_reg k2 + pipe(smem form)", F32, 30000, 2, dict(k_pass=[2], cr_levels=4, thomas_chains=32, tl_levels=3)),
    ("split_pipe k4 + pipe WL", F32, 1 << 17, 2, dict(k_pass=[4], cr_levels=4, thomas_chains=4, tl_levels=5)),
    ("split_pipe k7 (layout B) + pipe", F32, 1 << 20, 1, dict(k_pass=[7], cr_levels=4, thomas_chains=16, tl_levels=5)),
    ("split_pipe k8 256t", F32, 1 << 20, 1, dict(k_pass=[8], cr_levels=4, thomas_chains=8, tl_levels=5,
                                                  split_threads=256, split_tile_rows=4096)),
    ("two passes 4+3", F32, 300001, 2, dict(k_pass=[4, 3], cr_levels=2, thomas_chains=16, tl_levels=0)),
    ("split_pass k9 (smem tile)", F32, 200000, 1, dict(k_pass=[9], cr_levels=2, thomas_chains=8, tl_levels=0)),
    ("x_group 8", F32, 1 << 17, 2, dict(k_pass=[4], cr_levels=4, thomas_chains=1, tl_levels=5, x_group=8)),
    ("x_group 4", F32, 1 << 16, 2, dict(k_pass=[3], cr_levels=4, thomas_chains=1, tl_levels=5, x_group=4)),
    ("f64 k8 + pipe", F64, 1 << 20, 1, dict(k_pass=[8], cr_levels=3, thomas_chains=16, tl_levels=5)),
    ("f64 k0 cpipe C=2", F64, 8192, 2, dict(k_pass=[], cr_levels=3, thomas_chains=16, cluster=2, tl_levels=5)),
    ("f64 x_group 2", F64, 1 << 16, 2, dict(k_pass=[4], cr_levels=3, thomas_chains=1, tl_levels=5, x_group=2)),
    ("strided k3", F32, 65536, 2, dict(k_pass=[3], cr_levels=4, thomas_chains=1, tl_levels=5, strided=1)),
    ("f64 strided k2", F64, 9001, 2, dict(k_pass=[2], cr_levels=3, thomas_chains=1, tl_levels=5, strided=1)),
    ("coalesced k3 (global fallback)", F32, 65536, 2, dict(k_pass=[3], cr_levels=0, thomas_chains=64, tl_levels=0,
                                                          strided=2)),
    ("f64 coalesced k2", F64, 9000, 2, dict(k_pass=[2], cr_levels=0, thomas_chains=32, tl_levels=0, strided=2)),
]

bad = 0
# the interleaved layout (TMA transposer and the plain tile transposer)
for label, dt, n, m in [("interleaved TMA transpose", F32, 3000, 36), ("interleaved tile transpose", F32, 1000, 33)]:
    a, b, c, d = inputs.generate(n, m, dt, seed=6)
    plan = tds.Plan(n, m, "float32", device=0, mode="static")
    ti = [torch.from_numpy(np.ascontiguousarray(v.T)).cuda() for v in (a, b, c, d)]
    x = tds.solve_interleaved(plan, *ti).cpu().numpy().T
    err = oracle.rel_err(np.ascontiguousarray(x), oracle.thomas(a, b, c, d))
    ok = err <= 1e-4
    bad += not ok
    print(f"{'ok ' if ok else 'BAD'} {label}: n={n} m={m} rel_err={err:.2e}", flush=True)
for label, dt, n, m, params in CASES:
    a, b, c, d = inputs.generate(n, m, dt, seed=5)
    plan = tds.Plan(n, m, "float32" if dt == F32 else "float64", device=0, mode="static")
    if params:
        plan.set_params(**dict({"cluster": 1}, **params))
    ta, tb, tc, td = (torch.from_numpy(v).cuda() for v in (a, b, c, d))
    x = tds.solve_batched(plan, ta, tb, tc, td)
    torch.cuda.synchronize()
    err = oracle.rel_err(x.cpu().numpy(), oracle.thomas(a, b, c, d))
    ok = err <= (1e-4 if dt == F32 else 1e-10)
    bad += not ok
    print(f"{'ok ' if ok else 'BAD'} {label}: n={n} m={m} rel_err={err:.2e}", flush=True)
# round 2: device generator, the one-huge-system path in a loopback world (split to
# slots, normalised residue solves, exchange copies, x unpack), normalised solve
from paper_conf_ipps_davidsonzo11_b200 import dist as tdist  # noqa: E402
for label, dt, n, G, kd, chunks in [("huge loopback G=4 kd=3", F32, 1 << 16, 4, 3, 1),
                                    ("huge loopback G=2 kd=4 chunks=2", F64, 1 << 15, 2, 4, 2),
                                    ("huge G=1 kd=5", F32, 1 << 16, 1, 5, 1),
                                    ("huge loopback peer G=4 kd=3", F32, 1 << 16, 4, 3, 1),
                                    ("huge loopback peer G=2 kd=4", F64, 1 << 15, 2, 4, 1),
                                    ("huge loopback peer x-fused G=2 kd=3", F32, 1 << 23, 2, 3, 1)]:
    tdt = torch.float32 if dt == F32 else torch.float64
    name = "float32" if dt == F32 else "float64"
    be = tdist.CudaBackend(tdt, "cuda:0")
    ranks = [tdist.HugeRank(n, G, g, be, kd=kd, chunks=chunks) for g in range(G)]
    if "peer" in label:  # the split writes the residue classes straight into the owners (tds_split_scatter)
        for R in ranks:
            R.set_peers([P.sys_buf.data_ptr() for P in ranks])
    B = n // G
    for g, R in enumerate(ranks):
        tds.api.generate_rows(n, g * B, B, name, seed=5, out=R.local)
    outs = [be.empty(B) for _ in range(G)]
    tdist.solve_huge_loopback(ranks, outs)
    torch.cuda.synchronize()
    a, b, c, d = inputs.generate(n, 1, dt, seed=5)
    err = oracle.rel_err(torch.cat(outs).cpu().numpy()[None], oracle.thomas(a, b, c, d))
    ok = err <= (1e-4 if dt == F32 else 1e-10)
    bad += not ok
    print(f"{'ok ' if ok else 'BAD'} {label}: n={n} rel_err={err:.2e}", flush=True)
gen = tds.generate(3000, 5, "float64", seed=9, first_system=2)
torch.cuda.synchronize()
ref = inputs.generate(3000, 5, F64, seed=9, first_system=2)
ok = all(np.array_equal(r, g.cpu().numpy()) for r, g in zip(ref, gen))
bad += not ok
print(f"{'ok ' if ok else 'BAD'} tds_generate f64 bit-identical", flush=True)
sys.exit(1 if bad else 0)
