"""Multi-process tests of the multi-GPU decompositions on CPU (gloo,
world_size 2 and 4): the huge-system halo / all-to-all index arithmetic with
oracle-backed local compute, batch sharding and plan broadcast.  A 1-GPU test
runs the same huge-system path with the libtds kernels."""
import dataclasses
import os
import socket

import numpy as np
import pytest
import torch
import torch.distributed as dist
import torch.multiprocessing as mp

import oracle
from oracle import plan as rp
from paper_conf_ipps_davidsonzo11_b200 import inputs


def _free_port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


def cpu_split(a, b, c, d, kd):
    """Oracle k_d PCR levels, normalised (b' = 1), canonical residue order."""
    A, B, C, D = (v.detach().double().numpy()[None] for v in (a, b, c, d))
    sa, sb, sc, sd = oracle.pcr_split(A, B, C, D, kd)
    perm = oracle.permutation(A.shape[1], kd)
    return tuple(torch.from_numpy(np.ascontiguousarray(v[0, perm] / sb[0, perm])) for v in (sa, sc, sd))


def cpu_solve(a, b, c, d):
    return torch.from_numpy(oracle.thomas(a.numpy(), b.numpy(), c.numpy(), d.numpy()))


def _huge_worker(rank, world, port, n, kd, q):
    os.environ.update(MASTER_ADDR="127.0.0.1", MASTER_PORT=str(port))
    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        from paper_conf_ipps_davidsonzo11_b200 import dist as tdist
        a, b, c, d = inputs.generate(n, 1, np.float64, seed=31, mu=0.3)
        B = n // world
        sl = slice(rank * B, (rank + 1) * B)
        loc = [torch.from_numpy(np.ascontiguousarray(v[0, sl])) for v in (a, b, c, d)]
        x = tdist.solve_huge(*loc, n=n, kd=kd, split_fn=cpu_split, solve_fn=cpu_solve)
        xr = oracle.thomas(a, b, c, d)[0, sl]
        err = float(np.abs(x.numpy() - xr).max() / np.abs(xr).max())
        q.put((rank, err))
    finally:
        dist.destroy_process_group()


@pytest.mark.parametrize("world,n,kd", [(2, 4096, 1), (2, 4096, 3), (4, 8192, 2), (4, 8192, 4)])
def test_huge_system_gloo(world, n, kd):
    """One system split by row blocks over `world` gloo ranks: halo exchange,
    k_d local PCR levels, all-to-all of residue classes, local solves, x back.
    Must equal the single-process oracle solution."""
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    port = _free_port()
    procs = [ctx.Process(target=_huge_worker, args=(r, world, port, n, kd, q)) for r in range(world)]
    for p in procs:
        p.start()
    res = dict(q.get(timeout=120) for _ in range(world))
    for p in procs:
        p.join(60)
        assert p.exitcode == 0
    assert sorted(res) == list(range(world))
    assert max(res.values()) <= 1e-11, res


def _shard_worker(rank, world, port, q):
    os.environ.update(MASTER_ADDR="127.0.0.1", MASTER_PORT=str(port))
    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        import paper_conf_ipps_davidsonzo11_b200 as tds
        from paper_conf_ipps_davidsonzo11_b200 import dist as tdist
        props = dataclasses.asdict(rp.B200)
        plan = tds.Plan(1 << 20, 16, "float32", props=props, mode="static")
        if rank == 0:  # e.g. a tuned plan: only rank 0 knows it
            plan.set_params(k_pass=[4, 3], cluster=1, tl_levels=0, cr_levels=4, thomas_chains=64)
        tdist.broadcast_plan(plan, src=0)
        ranges = [tdist.shard_range(37, world, r) for r in range(world)]
        # generator: the rank's shard equals the rows of the unsharded batch
        s0, s1 = ranges[rank]
        _, _, _, dsh = inputs.generate(1000, s1 - s0, np.float32, seed=4, first_system=s0)
        _, _, _, dall = inputs.generate(1000, 37, np.float32, seed=4)
        q.put((rank, plan.params_list(), ranges, bool(np.array_equal(dsh, dall[s0:s1]))))
    finally:
        dist.destroy_process_group()


def test_batch_sharding_gloo():
    world = 2
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    port = _free_port()
    procs = [ctx.Process(target=_shard_worker, args=(r, world, port, q)) for r in range(world)]
    for p in procs:
        p.start()
    out = {r: (pl, rg, eq) for r, pl, rg, eq in (q.get(timeout=120) for _ in range(world))}
    for p in procs:
        p.join(60)
        assert p.exitcode == 0
    assert out[0][0] == out[1][0]            # identical integer plans on every rank
    rg = out[0][1]
    assert rg[0][0] == 0 and rg[-1][1] == 37 and all(rg[i][1] == rg[i + 1][0] for i in range(world - 1))
    assert out[0][2] and out[1][2]


def test_huge_bytes_accounting():
    from paper_conf_ipps_davidsonzo11_b200 import dist as tdist
    b = tdist.huge_bytes(1 << 28, 8)
    assert b["all_to_all_split"] == 3 * (1 << 25) * 4 * 7 // 8


@pytest.mark.gpu
def test_huge_system_single_gpu_kernels():
    """The huge-system path (G = 1) with the libtds split-only plan and solve."""
    from paper_conf_ipps_davidsonzo11_b200 import dist as tdist
    n = 1 << 20
    a, b, c, d = inputs.generate(n, 1, np.float32, seed=5)
    loc = [torch.from_numpy(v[0].copy()).cuda() for v in (a, b, c, d)]
    x = tdist.solve_huge(*loc, n=n, kd=4)
    torch.cuda.synchronize()
    xr = oracle.thomas(a, b, c, d)[0]
    assert np.abs(x.cpu().numpy() - xr).max() / np.abs(xr).max() <= 1e-4


@pytest.mark.gpu
@pytest.mark.parametrize("n,m,params", [
    (1 << 20, 8, dict(k_pass=[7], cr_levels=4, thomas_chains=16, cluster=1, tl_levels=5)),
    (16384, 96, dict(k_pass=[], cr_levels=4, thomas_chains=32, cluster=2, tl_levels=5)),
    (65536, 24, dict(k_pass=[], cr_levels=4, thomas_chains=16, cluster=8, tl_levels=5))],
    ids=["cfg3-shape", "cfg4-shape", "cfg2-shape"])
@pytest.mark.parametrize("world", [2, 3, 8])
def test_batch_shards_bit_identical_gpu(n, m, params, world):
    """SURVEY §8(c) "Sharding": x of every rank's shard (its own Plan(n, m_rank)
    with the broadcast integer plan, inputs generated with global system
    indices) is bit-identical to the same systems of the unsharded solve."""
    import paper_conf_ipps_davidsonzo11_b200 as tds
    from paper_conf_ipps_davidsonzo11_b200 import dist as tdist
    a, b, c, d = inputs.generate(n, m, np.float32, seed=11)
    full = tds.Plan(n, m, "float32", device=0)
    full.set_params(**params)
    xall = tds.solve_batched(full, *[torch.from_numpy(v).cuda() for v in (a, b, c, d)]).cpu().numpy()
    for r in range(world):
        s0, s1 = tdist.shard_range(m, world, r)
        if s1 <= s0:
            continue
        sh = inputs.generate(n, s1 - s0, np.float32, seed=11, first_system=s0)
        plan = tds.Plan(n, s1 - s0, "float32", device=0)
        plan.set_params_list(full.params_list())
        x = tds.solve_batched(plan, *[torch.from_numpy(v).cuda() for v in sh]).cpu().numpy()
        assert np.array_equal(x, xall[s0:s1])
