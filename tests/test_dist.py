"""Multi-process tests of the multi-GPU decompositions on CPU (gloo,
world_size 2 and 4): the huge-system halo / all-to-all index arithmetic with
oracle-backed local compute, batch sharding and plan broadcast.  A 1-GPU test
runs the same huge-system path with the libtds kernels."""
import ctypes
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


class OracleBackend:
    """solve_huge's local compute on the CPU oracle (test infrastructure): the
    split by oracle.pcr_split (normalised, canonical residue slots), the
    residue systems by fp64 Thomas, the unpack by a transpose."""

    def __init__(self, dtype=torch.float64):
        self.dtype = dtype

    def empty(self, *shape):
        return torch.empty(*shape, dtype=self.dtype)

    def make_split(self, E, kd):
        NR = 1 << kd
        assert E % NR == 0
        buf = torch.empty(3, NR, E // NR, dtype=self.dtype)
        return kd, buf, (buf[0], buf[1], buf[2])

    def split(self, state, ext):
        kd, buf, _ = state
        E = ext.shape[1]
        A, B, C, D = (ext[t].double().numpy()[None] for t in range(4))
        sa, sb, sc, sd = oracle.pcr_split(A, B, C, D, kd)
        perm = oracle.permutation(E, kd)
        for t, v in enumerate((sa, sc, sd)):
            buf[t] = torch.from_numpy((v[0, perm] / sb[0, perm]).reshape(buf.shape[1], buf.shape[2]))

    def make_solve(self, NL, m, stride):
        return NL, m, stride

    def solve(self, state, a, c, d, x):
        NL, m, stride = state
        view = (lambda t: torch.as_strided(t, (m, NL), (stride, 1))) if a.dim() == 1 else (lambda t: t)
        A, C, D = (view(t).double().numpy() for t in (a, c, d))
        x[:, :NL].copy_(torch.from_numpy(oracle.thomas(A, np.ones_like(A), C, D)))

    def unpack(self, xs, out, B, kd, slot_rows):
        NR = 1 << kd
        out.copy_(xs[:, :B // NR].t().reshape(B))


def _huge_worker(rank, world, port, n, kd, chunks, q):
    os.environ.update(MASTER_ADDR="127.0.0.1", MASTER_PORT=str(port))
    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        from paper_conf_ipps_davidsonzo11_b200 import dist as tdist
        a, b, c, d = inputs.generate(n, 1, np.float64, seed=31, mu=0.3)
        B = n // world
        sl = slice(rank * B, (rank + 1) * B)
        loc = [torch.from_numpy(np.ascontiguousarray(v[0, sl])) for v in (a, b, c, d)]
        x = tdist.solve_huge(*loc, n=n, kd=kd, backend=OracleBackend(), chunks=chunks)
        xr = oracle.thomas(a, b, c, d)[0, sl]
        err = float(np.abs(x.numpy() - xr).max() / np.abs(xr).max())
        q.put((rank, err, x.numpy().tobytes()))
    finally:
        dist.destroy_process_group()


@pytest.mark.parametrize("world,n,kd,chunks", [(2, 4096, 1, 1), (2, 4096, 3, 2), (4, 8192, 2, 1), (4, 8192, 4, 4)])
def test_huge_system_gloo(world, n, kd, chunks):
    """One system split by row blocks over `world` gloo ranks (point-to-point
    ops, the NCCL pattern): halo exchange into the padding, k_d PCR levels,
    all-to-all of residue slot segments (chunked), residue solves, x back,
    unpack.  Must equal the single-process oracle solution, and bit-equal the
    same solve in a one-process loopback world."""
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    port = _free_port()
    procs = [ctx.Process(target=_huge_worker, args=(r, world, port, n, kd, chunks, q)) for r in range(world)]
    for p in procs:
        p.start()
    res = {r: (e, xb) for r, e, xb in (q.get(timeout=120) for _ in range(world))}
    for p in procs:
        p.join(60)
        assert p.exitcode == 0
    assert sorted(res) == list(range(world))
    assert max(e for e, _ in res.values()) <= 1e-11, res
    xs = _loopback_cpu(n, world, kd, chunks)
    for r in range(world):
        assert xs[r].numpy().tobytes() == res[r][1]


def _loopback_cpu(n, G, kd, chunks, seed=31):
    from paper_conf_ipps_davidsonzo11_b200 import dist as tdist
    a, b, c, d = inputs.generate(n, 1, np.float64, seed=seed, mu=0.3)
    be = OracleBackend()
    ranks = [tdist.HugeRank(n, G, g, be, kd=kd, chunks=chunks) for g in range(G)]
    B = n // G
    for g, R in enumerate(ranks):
        for dst, v in zip(R.local, (a, b, c, d)):
            dst.copy_(torch.from_numpy(v[0, g * B:(g + 1) * B]))
    outs = [be.empty(B) for _ in range(G)]
    return tdist.solve_huge_loopback(ranks, outs)


@pytest.mark.parametrize("kd,chunks", [(3, 1), (3, 2), (4, 1)])
def test_huge_loopback_cpu_bit_identical_over_G(kd, chunks):
    """The loopback world (G ranks in one process): x is the oracle's, and
    bit-identical for G = 1, 2, 4, 8 (every row's split coefficients come from
    the same operands whatever the block boundaries; the residue systems are
    the same)."""
    n = 4096
    a, b, c, d = inputs.generate(n, 1, np.float64, seed=31, mu=0.3)
    xr = oracle.thomas(a, b, c, d)[0]
    ref = None
    for G in (1, 2, 4, 8):
        if (1 << kd) % G or (1 << kd) // G % chunks:
            continue
        x = torch.cat(_loopback_cpu(n, G, kd, chunks)).numpy()
        assert np.abs(x - xr).max() <= 1e-11 * np.abs(xr).max()
        if ref is None:
            ref = x
        assert np.array_equal(x, ref), G


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
    """NVLink bytes per rank: config 5 at 8 GPUs moves 3 split
    arrays x 7/8 of its 2^25 rows (~ 352 MB) out and in, and 7/8 of its x
    (~ 117 MB) back."""
    from paper_conf_ipps_davidsonzo11_b200 import dist as tdist
    b = tdist.huge_bytes(1 << 28, 8, kd=8)
    assert b["all_to_all_split"] == 3 * (1 << 25) * 4 * 7 // 8
    assert b["all_to_all_x"] == (1 << 25) * 4 * 7 // 8
    assert b["halo"] == 2 * 4 * 1024 * 4


@pytest.mark.gpu
def test_huge_system_single_gpu_kernels():
    """The huge-system path (G = 1, torch.distributed not initialised) with
    the libtds kernels: split to slots, residue systems read in place."""
    from paper_conf_ipps_davidsonzo11_b200 import dist as tdist
    n = 1 << 20
    a, b, c, d = inputs.generate(n, 1, np.float32, seed=5)
    loc = [torch.from_numpy(v[0].copy()).cuda() for v in (a, b, c, d)]
    x = tdist.solve_huge(*loc, n=n, kd=4)
    torch.cuda.synchronize()
    xr = oracle.thomas(a, b, c, d)[0]
    assert np.abs(x.cpu().numpy() - xr).max() / np.abs(xr).max() <= 1e-4


def _loopback_gpu(n, G, kd, chunks, dtype, seed=5):
    from paper_conf_ipps_davidsonzo11_b200 import dist as tdist
    tdt = torch.float32 if dtype == np.float32 else torch.float64
    be = tdist.CudaBackend(tdt, "cuda:0")
    ranks = [tdist.HugeRank(n, G, g, be, kd=kd, chunks=chunks) for g in range(G)]
    B = n // G
    import paper_conf_ipps_davidsonzo11_b200 as tds
    for g, R in enumerate(ranks):  # each rank draws its own rows (device generator, global row index)
        tds.api.generate_rows(n, g * B, B, "float32" if dtype == np.float32 else "float64", seed=seed, out=R.local)
    outs = [be.empty(B) for _ in range(G)]
    tdist.solve_huge_loopback(ranks, outs)
    torch.cuda.synchronize()
    return torch.cat(outs).cpu().numpy()


@pytest.mark.gpu
@pytest.mark.parametrize("dtype", [np.float32, np.float64])
@pytest.mark.parametrize("kd,chunks", [(3, 1), (5, 4), (8, 8)])
def test_huge_loopback_gpu(dtype, kd, chunks):
    """The whole multi-rank huge-system data path on ONE GPU (G = 1, 2, 4, 8
    ranks in a loopback world, libtds kernels, messages as device copies):
    the oracle's x within the tolerance and bit-identical for every G."""
    n = 1 << 20
    a, b, c, d = inputs.generate(n, 1, dtype, seed=5)
    xr = oracle.thomas(a, b, c, d)[0]
    ref = None
    for G in (1, 2, 4, 8):
        if (1 << kd) % G or (1 << kd) // G % chunks:
            continue
        x = _loopback_gpu(n, G, kd, chunks, dtype)
        err = np.abs(x - xr).max() / np.abs(xr).max()
        assert err <= (1e-4 if dtype == np.float32 else 1e-10), (G, err)
        if ref is None:
            ref = x
        assert np.array_equal(x, ref), G


@pytest.mark.gpu
@pytest.mark.parametrize("dtype", [np.float32, np.float64])
@pytest.mark.parametrize("n,kp", [(4096 + 256, [3]), (1 << 20, [8]), (100000, [5]), (1 << 18, [4, 4])])
def test_split_slots_pack_bit_exact(dtype, n, kp):
    """G3 pack: tds_split_slots leaves residue r of system s in slot (s << k) + r
    -- the same numbers, bit for bit, as the canonical diagnostic split
    (tds_split_batched) in the torch reference layout."""
    import paper_conf_ipps_davidsonzo11_b200 as tds
    name = "float32" if dtype == np.float32 else "float64"
    m = 2
    dv = [torch.from_numpy(v).cuda() for v in inputs.generate(n, m, dtype, seed=3)]
    plan = tds.Plan(n, m, name, device=0)
    plan.set_params(k_pass=kp, split_only=1, cluster=1, tl_levels=0)
    ref = tds.split_batched(plan, *dv)
    ws = plan.workspace()
    views = tds.api.split_slots(plan, *dv, workspace=ws)
    torch.cuda.synchronize()
    k = sum(kp)
    NR = 1 << k
    lay = plan.slots_layout()
    assert lay["num_slots"] == m * NR and lay["slot_rows"] >= -(-n // NR)
    for v, r_ in zip(views, ref):
        off = 0
        for r in range(NR):
            L = -(-(n - r) // NR)
            for s in range(m):
                assert torch.equal(v[s * NR + r, :L], r_[s, off:off + L])
            off += L


@pytest.mark.gpu
@pytest.mark.parametrize("dtype", [np.float32, np.float64])
@pytest.mark.parametrize("n,m,k,slot", [(1 << 16, 3, 5, 2048), (1 << 16, 1, 8, 256), (5000, 2, 2, 1260),
                                        (4096, 2, 6, 96)])
def test_unpack_residues_bit_exact(dtype, n, m, k, slot):
    """G3 unpack: tds_unpack_residues is the residue -> row transpose of the
    torch reference: x[s, r + 2^k j] = xs[(s << k) + r, j]; xs left intact."""
    import paper_conf_ipps_davidsonzo11_b200 as tds
    tdt = torch.float32 if dtype == np.float32 else torch.float64
    NR = 1 << k
    xs = torch.randn(m * NR, slot, dtype=tdt, device="cuda")
    keep = xs.clone()
    x = torch.full((m, n), 7.0, dtype=tdt, device="cuda")
    tds.api.unpack_residues(xs, x, n, m, k, slot)
    torch.cuda.synchronize()
    ref = torch.empty(m, n, dtype=tdt, device="cuda")
    for r in range(NR):
        L = -(-(n - r) // NR)
        ref[:, r::NR] = xs.view(m, NR, slot)[:, r, :L]
    assert torch.equal(x, ref) and torch.equal(xs, keep)


@pytest.mark.gpu
@pytest.mark.parametrize("dtype", [np.float32, np.float64])
@pytest.mark.parametrize("n,m,params", [(1 << 20, 4, dict(k_pass=[7], cr_levels=4, thomas_chains=1, tl_levels=5)),
                                        (100000, 3, dict(k_pass=[5], cr_levels=3, thomas_chains=32, tl_levels=0)),
                                        (1 << 18, 2, dict(k_pass=[3, 3], cr_levels=4, thomas_chains=1, tl_levels=5))])
def test_solve_normalized_equals_b_one(dtype, n, m, params):
    """tds_solve_normalized (no b array) is bit-identical to tds_solve_batched
    with a materialised b = 1 (normalising by rcp(1) = 1 is exact)."""
    import paper_conf_ipps_davidsonzo11_b200 as tds
    name = "float32" if dtype == np.float32 else "float64"
    if dtype == np.float64:  # R_max = 8: subsystems of <= 4096 rows
        params = dict(params, cr_levels=3, k_pass=[k + 1 for k in params["k_pass"][:1]] + params["k_pass"][1:])
    a, b, c, d = inputs.generate(n, m, dtype, seed=8)
    an, cn, dn = (v / b for v in (a, c, d))
    ta, tc, td = (torch.from_numpy(np.ascontiguousarray(v)).cuda() for v in (an, cn, dn))
    plan = tds.Plan(n, m, name, device=0)
    plan.set_params(cluster=1, **params)
    x1 = tds.api.solve_normalized(plan, ta, tc, td)
    x2 = tds.solve_batched(plan, ta, torch.ones_like(ta), tc, td)
    torch.cuda.synchronize()
    assert torch.equal(x1, x2)
    xr = oracle.thomas(an, np.ones_like(an), cn, dn)
    assert oracle.rel_err(x1.cpu().numpy(), xr) <= (1e-4 if dtype == np.float32 else 1e-10)


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


@pytest.mark.gpu
def test_huge_tuned_residue_plan(tmp_path):
    """The residue solves with a tds_tune'd plan (bench.py --config 5 tunes
    it on rank 0 and broadcasts it): same x as the static plan within the
    tolerance, and every chunk runs the same integer plan."""
    from paper_conf_ipps_davidsonzo11_b200 import dist as tdist
    import paper_conf_ipps_davidsonzo11_b200 as tds
    n, kd = 1 << 20, 5
    be = tdist.CudaBackend(torch.float32, "cuda:0")
    R = tdist.HugeRank(n, 1, 0, be, kd=kd, chunks=2)
    vals = R.tune_residues(cache_path=str(tmp_path / "t.txt"))
    assert all(p.params_list() == vals for p, _ in R.solve_states)
    tds.api.generate_rows(n, 0, n, "float32", seed=5, out=R.local)
    out = be.empty(n)
    tdist.solve_huge_loopback([R], [out])
    torch.cuda.synchronize()
    a, b, c, d = inputs.generate(n, 1, np.float32, seed=5)
    xr = oracle.thomas(a, b, c, d)[0]
    assert np.abs(out.cpu().numpy() - xr).max() / np.abs(xr).max() <= 1e-4


@pytest.mark.gpu
@pytest.mark.parametrize("family,kw", [("poisson", {}), ("const", {"param": 1e-6})])
@pytest.mark.parametrize("kd,chunks", [(3, 1), (5, 2)])
def test_huge_loopback_gpu_coupling(family, kw, kd, chunks):
    """The multi-rank huge-system path on long-range-coupled fp64 systems
    (every row couples to rows on every other rank): the halo exchange, the
    residue all-to-all and the x return must carry the coupling.  Oracle
    within 10 kappa eps_64, bit-identical over G = 1, 2, 4, 8."""
    import math
    from paper_conf_ipps_davidsonzo11_b200 import dist as tdist
    n = 1 << 18
    a, b, c, d = inputs.generate(n, 1, np.float64, seed=7, family=family, **kw)
    xr = oracle.thomas(a, b, c, d)[0]
    delta = kw.get("param", 0.0)
    cs = math.cos(math.pi / (n + 1))
    kappa = (2 + delta + 2 * cs) / (2 + delta - 2 * cs)
    be = tdist.CudaBackend(torch.float64, "cuda:0")
    ref = None
    for G in (1, 2, 4, 8):
        if (1 << kd) % G or (1 << kd) // G % chunks:
            continue
        B = n // G
        ranks = [tdist.HugeRank(n, G, g, be, kd=kd, chunks=chunks) for g in range(G)]
        for g, R in enumerate(ranks):
            for dst, v in zip(R.local, (a, b, c, d)):
                dst.copy_(torch.from_numpy(v[0, g * B:(g + 1) * B]))
        outs = [be.empty(B) for _ in range(G)]
        tdist.solve_huge_loopback(ranks, outs)
        torch.cuda.synchronize()
        x = torch.cat(outs).cpu().numpy()
        err = np.abs(x - xr).max() / np.abs(xr).max()
        assert err <= 10 * kappa * 2.22e-16, (G, err)
        if ref is None:
            ref = x
        assert np.array_equal(x, ref), G


@pytest.mark.gpu
@pytest.mark.parametrize("stride_pad,kp", [(3, [3]), (3, [6]), (16, [7]), (5, [4, 3])])
def test_solve_normalized_padded_strides(stride_pad, kp):
    """tds_solve_normalized with a padded (and for odd pads, non-16-byte)
    batch stride: the register / shared-memory split kernels read the
    normalised caller arrays; equal to the materialised-b = 1 solve and the
    oracle; the padding is untouched."""
    import paper_conf_ipps_davidsonzo11_b200 as tds
    n, m = 50000, 3
    stride = n + stride_pad
    a, b, c, d = inputs.generate(n, m, np.float32, seed=12)
    an, cn, dn = (v / b for v in (a, c, d))
    pad = lambda v: np.pad(v, ((0, 0), (0, stride_pad)), constant_values=7.0).reshape(-1)
    ta, tc, td = (torch.from_numpy(pad(v)).cuda() for v in (an, cn, dn))
    plan = tds.Plan(n, m, "float32", device=0, batch_stride=stride)
    R = 16 if -(-n // (1 << sum(kp))) > 4096 else 8
    plan.set_params(k_pass=kp, cluster=1, cr_levels=R.bit_length() - 1, thomas_chains=1, tl_levels=5)
    out = torch.full_like(td, 7.0)
    tds.api.solve_normalized(plan, ta, tc, td, out=out)
    x2 = tds.solve_batched(plan, ta, torch.ones_like(ta), tc, td)
    torch.cuda.synchronize()
    xs = out.cpu().numpy().reshape(m, stride)
    assert np.all(xs[:, n:] == 7.0)
    assert np.array_equal(xs[:, :n], x2.cpu().numpy().reshape(m, stride)[:, :n])
    xr = oracle.thomas(an, np.ones_like(an), cn, dn)
    assert oracle.rel_err(xs[:, :n], xr) <= 1e-4


# ------------------------------------------- peer mode: the all-to-all fused into the split

def _peer_ranks(n, G, kd, chunks, dtype, seed=5, family="dd", kw=None):
    from paper_conf_ipps_davidsonzo11_b200 import dist as tdist
    import paper_conf_ipps_davidsonzo11_b200 as tds
    tdt = torch.float32 if dtype == np.float32 else torch.float64
    be = tdist.CudaBackend(tdt, "cuda:0")
    ranks = [tdist.HugeRank(n, G, g, be, kd=kd, chunks=chunks) for g in range(G)]
    for R in ranks:  # every rank writes straight into its peers' residue buffers (one device here)
        R.set_peers([P.sys_buf.data_ptr() for P in ranks])
    B = n // G
    if family == "dd":
        for g, R in enumerate(ranks):
            tds.api.generate_rows(n, g * B, B, "float32" if dtype == np.float32 else "float64", seed=seed,
                                  out=R.local)
    else:
        a, b, c, d = inputs.generate(n, 1, dtype, seed=seed, family=family, **(kw or {}))
        for g, R in enumerate(ranks):
            for dst, v in zip(R.local, (a, b, c, d)):
                dst.copy_(torch.from_numpy(v[0, g * B:(g + 1) * B]))
    outs = [be.empty(B) for _ in range(G)]
    tdist.solve_huge_loopback(ranks, outs)
    torch.cuda.synchronize()
    return torch.cat(outs).cpu().numpy()


@pytest.mark.gpu
@pytest.mark.parametrize("dtype", [np.float32, np.float64])
@pytest.mark.parametrize("G,kd,chunks", [(2, 3, 1), (4, 5, 2), (8, 8, 4)])
def test_huge_peer_mode_loopback(dtype, G, kd, chunks):
    """Peer mode (tds_split_scatter: every rank's split writes each residue
    class straight into its owner's buffer, then a barrier): bit-identical to
    the point-to-point all-to-all and to G = 1, and the oracle's x."""
    n = 1 << 20
    x = _peer_ranks(n, G, kd, chunks, dtype)
    assert np.array_equal(x, _loopback_gpu(n, G, kd, chunks, dtype))
    assert np.array_equal(x, _loopback_gpu(n, 1, kd, 1, dtype))
    a, b, c, d = inputs.generate(n, 1, dtype, seed=5)
    xr = oracle.thomas(a, b, c, d)[0]
    assert np.abs(x - xr).max() / np.abs(xr).max() <= (1e-4 if dtype == np.float32 else 1e-10)


@pytest.mark.gpu
def test_huge_peer_mode_coupling():
    """Peer mode on the Poisson matrix (every row couples across ranks)."""
    import math
    n, G, kd = 1 << 18, 4, 5
    x = _peer_ranks(n, G, kd, 1, np.float64, seed=7, family="poisson")
    a, b, c, d = inputs.generate(n, 1, np.float64, seed=7, family="poisson")
    xr = oracle.thomas(a, b, c, d)[0]
    cs = math.cos(math.pi / (n + 1))
    kappa = (2 + 2 * cs) / (2 - 2 * cs)
    assert np.abs(x - xr).max() / np.abs(xr).max() <= 10 * kappa * 2.22e-16


@pytest.mark.gpu
@pytest.mark.parametrize("dtype", [np.float32, np.float64])
@pytest.mark.parametrize("E,kd,G,off,num", [(4096 + 256, 3, 2, 4, 500), ((1 << 18) + 4096, 8, 8, 8, 1024),
                                            (65536, 5, 4, 4, 2040)])
def test_split_scatter_bit_exact(dtype, E, kd, G, off, num):
    """tds_split_scatter writes residue h q + rl, positions [off, off + num),
    to dst[t][h] + rl * stride: the same bits as the canonical split slots;
    everything else in the destinations untouched (the halo positions are
    clipped by the TMA stores)."""
    import paper_conf_ipps_davidsonzo11_b200 as tds
    name = "float32" if dtype == np.float32 else "float64"
    tdt = torch.float32 if dtype == np.float32 else torch.float64
    dv = [torch.from_numpy(v).cuda() for v in inputs.generate(E, 1, dtype, seed=4)]
    plan = tds.Plan(E, 1, name, device=0)
    plan.set_params(k_pass=[kd], split_only=1, cluster=1, tl_levels=0)
    views = tds.api.split_slots(plan, *dv, workspace=plan.workspace())
    NR, q = 1 << kd, (1 << kd) // G
    stride = -(-(num + 3) // 4) * 4
    dst = [[torch.full((q, stride), 7.0, dtype=tdt, device="cuda") for _ in range(G)] for _ in range(3)]
    tds.api.split_scatter(plan, *dv, dst, q, off, num, stride)
    torch.cuda.synchronize()
    for t in range(3):
        for h in range(G):
            got = dst[t][h]
            assert torch.equal(got[:, :num], views[t][h * q:(h + 1) * q, off:off + num])
            assert bool((got[:, num:] == 7.0).all())


def test_split_scatter_argument_errors():
    """Rejected before anything is enqueued (plan from fake B200 properties)."""
    import paper_conf_ipps_davidsonzo11_b200 as tds
    from paper_conf_ipps_davidsonzo11_b200 import _lib as L
    lib = L.load()
    p = tds.Plan(4096, 1, "float32", props=dataclasses.asdict(rp.B200))
    p.set_params(k_pass=[3], split_only=1, cluster=1, tl_levels=0)
    spec = L.Scatter()
    spec.groups, spec.residues_per_group, spec.first_pos, spec.num_pos, spec.dst_stride = 2, 4, 0, 100, 128
    for t in range(3):
        for h in range(2):
            spec.dst[t][h] = (1 << 40) + (t * 2 + h) * (1 << 20)
    A = 1 << 36
    call = lambda: lib.tds_split_scatter(p.handle, A, A + (1 << 24), A + (2 << 24), A + (3 << 24),
                                         ctypes.byref(spec), None)
    assert call() in (5, 7)                      # valid: fails only at the device check (no GPU / no device)
    spec.residues_per_group = 3
    assert call() == 1                           # groups * q != 2^k
    spec.residues_per_group = 4
    spec.dst_stride = 50
    assert call() == 1                           # dst_stride < num_pos
    spec.dst_stride = 128
    spec.num_pos = 1000
    assert call() == 1                           # window past floor(n / 2^k) = 512
    spec.num_pos = 100
    spec.first_pos = 2
    assert call() == 1                           # first_pos not a 16-byte multiple (fp32: 4 elements)
    spec.first_pos = 0
    spec.num_pos = 98
    assert call() == 1                           # num_pos not a 16-byte multiple
    spec.num_pos = 100
    spec.dst[1][1] = (1 << 40) + 8
    assert call() == 1                           # misaligned dst
    q2 = tds.Plan(4096, 2, "float32", props=dataclasses.asdict(rp.B200))
    q2.set_params(k_pass=[3], split_only=1, cluster=1, tl_levels=0)
    assert lib.tds_split_scatter(q2.handle, A, A, A, A, ctypes.byref(spec), None) == 2  # m != 1


@pytest.mark.gpu
@pytest.mark.parametrize("dtype", [np.float32, np.float64])
@pytest.mark.parametrize("G,kd", [(2, 3), (4, 4)])
def test_huge_peer_mode_x_fused(dtype, G, kd):
    """Peer mode with BOTH exchanges fused: the split's stores scatter the
    residue classes, the residue solves' placement writes x straight into its
    owners (tds_solve_normalized_xscatter).  Bit-identical to the
    point-to-point path, the oracle's x."""
    from paper_conf_ipps_davidsonzo11_b200 import dist as tdist
    n = 1 << 24
    tdt = torch.float32 if dtype == np.float32 else torch.float64
    be = tdist.CudaBackend(tdt, "cuda:0")
    probe = tdist.HugeRank(n, G, 0, be, kd=kd)
    probe.set_peers([probe.sys_buf.data_ptr()] * G)
    assert probe.x_fused, (probe.solve_states[0][0].info["k"], probe.Bj)
    del probe
    x = _peer_ranks(n, G, kd, 1, dtype)
    assert np.array_equal(x, _loopback_gpu(n, G, kd, 1, dtype))
    a, b, c, d = inputs.generate(n, 1, dtype, seed=5)
    xr = oracle.thomas(a, b, c, d)[0]
    assert np.abs(x - xr).max() / np.abs(xr).max() <= (1e-4 if dtype == np.float32 else 1e-10)


@pytest.mark.gpu
@pytest.mark.parametrize("dtype", [np.float32, np.float64])
def test_solve_normalized_xscatter_bit_exact(dtype):
    """x rows [h R, (h+1) R) of system s land at dst[h] + s * stride, the same
    bits as tds_solve_normalized; nothing else written."""
    import paper_conf_ipps_davidsonzo11_b200 as tds
    n, m, G = 1 << 20, 3, 4
    R = n // G
    tdt = torch.float32 if dtype == np.float32 else torch.float64
    a, b, c, d = inputs.generate(n, m, dtype, seed=21)
    an, cn, dn = (torch.from_numpy(np.ascontiguousarray(v / b)).cuda() for v in (a, c, d))
    plan = tds.Plan(n, m, "float32" if dtype == np.float32 else "float64", device=0)
    plan.set_params(k_pass=[7] if dtype == np.float32 else [8], cluster=1,
                    cr_levels=4 if dtype == np.float32 else 3, thomas_chains=1, tl_levels=5)
    xref = tds.api.solve_normalized(plan, an, cn, dn)
    stride = R + 64
    dst = [torch.full((m, stride), 7.0, dtype=tdt, device="cuda") for _ in range(G)]
    tds.api.solve_normalized_xscatter(plan, an, cn, dn, dst, R, stride)
    torch.cuda.synchronize()
    for h in range(G):
        assert torch.equal(dst[h][:, :R], xref[:, h * R:(h + 1) * R])
        assert bool((dst[h][:, R:] == 7.0).all())


def test_solve_xscatter_argument_errors():
    """tds_solve_normalized_xscatter's shape rules, before anything is enqueued."""
    import paper_conf_ipps_davidsonzo11_b200 as tds
    from paper_conf_ipps_davidsonzo11_b200 import _lib as L
    lib = L.load()
    p = tds.Plan(1 << 20, 2, "float32", props=dataclasses.asdict(rp.B200))
    p.set_params(k_pass=[7], cluster=1, cr_levels=4, thomas_chains=1, tl_levels=5)
    spec = L.XScatter()
    spec.groups, spec.rows_per_group, spec.dst_system_stride = 4, 1 << 18, 1 << 18
    for h in range(4):
        spec.dst[h] = (1 << 40) + h * (1 << 24)
    A, W = 1 << 36, 1 << 38
    ws = p.workspace_bytes
    call = lambda plan=p: lib.tds_solve_normalized_xscatter(plan.handle, A, A + (1 << 26), A + (2 << 26),
                                                            ctypes.byref(spec), W, ws, None)
    assert call() in (5, 7)                     # valid: fails only at the device check
    spec.rows_per_group = 1 << 17
    assert call() == 1                          # groups * rows_per_group != n
    spec.rows_per_group, spec.groups = 1 << 19, 2
    spec.dst_system_stride = (1 << 19) - 4
    assert call() == 1                          # stride < rows_per_group
    spec.dst_system_stride = 1 << 19
    assert call() in (5, 7)
    spec.dst[1] = (1 << 40) + 8
    assert call() == 1                          # misaligned destination
    spec.dst[1] = (1 << 40) + (1 << 24)
    q = tds.Plan(65536, 2, "float32", props=dataclasses.asdict(rp.B200))
    q.set_params(k_pass=[3], cluster=1, cr_levels=4, thomas_chains=1, tl_levels=5)
    spec.groups, spec.rows_per_group, spec.dst_system_stride = 2, 32768, 32768
    assert lib.tds_solve_normalized_xscatter(q.handle, A, A + (1 << 26), A + (2 << 26), ctypes.byref(spec), W,
                                             q.workspace_bytes, None) == 2  # k < 5: no TMA placement
