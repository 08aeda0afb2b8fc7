"""GPU parity: the CUDA path (through the C ABI) against the CPU oracle on the
same seeded inputs.  Tolerances (BASELINE.json north_star; R17):
fp32 normwise relative error <= 1e-4 and residual <= 1e-5; fp64 relative
error <= 1e-10.  Integer/index outputs (permutation, split structure) bit-exact."""
import math

import numpy as np
import pytest

import oracle
from paper_conf_ipps_davidsonzo11_b200 import inputs

pytestmark = pytest.mark.gpu

TOL = {np.float32: (1e-4, 1e-5), np.float64: (1e-10, 1e-12)}


@pytest.fixture(scope="module")
def tds():
    import torch
    assert torch.cuda.is_available()
    import paper_conf_ipps_davidsonzo11_b200 as m
    m._lib.load()
    return m


def to_dev(*arrs):
    import torch
    return [torch.from_numpy(np.ascontiguousarray(v)).cuda() for v in arrs]


def run(tds, a, b, c, d, mode="static", params=None, stride=0, inplace=False):
    import torch
    m, n = d.shape
    dt = "float32" if d.dtype == np.float32 else "float64"
    plan = tds.Plan(n, m, dt, device=0, mode=mode)
    if params:
        plan.set_params(**dict({"cluster": 1, "tl_levels": 0}, **params))
    ta, tb, tc, td = to_dev(a, b, c, d)
    x = tds.solve_batched(plan, ta, tb, tc, td, out=td if inplace else None)
    torch.cuda.synchronize()
    return x.cpu().numpy(), plan


def check(a, b, c, d, x, dtype, xr=None):
    if xr is None:
        xr = oracle.thomas(a, b, c, d)
    err = oracle.rel_err(x, xr)
    etol, rtol = TOL[dtype]
    assert np.all(np.isfinite(x))
    assert err <= etol, f"rel_err {err:.3e} > {etol}"
    if dtype == np.float32:
        res = oracle.residual(a, b, c, d, x)
        assert res <= rtol, f"residual {res:.3e} > {rtol}"
    return err


# ------------------------------------------------ on-chip kernel alone (k = 0)

@pytest.mark.parametrize("dtype", [np.float32, np.float64])
@pytest.mark.parametrize("n", [1, 2, 3, 31, 32, 33, 100, 1000, 1024, 4097, 8192])
def test_onchip_k0_static(tds, dtype, n):
    if dtype == np.float64 and n > 4096:
        n = 4096
    a, b, c, d = inputs.generate(n, 5, dtype, seed=21)
    x, plan = run(tds, a, b, c, d, params=None)
    assert plan.info["k"] == 0
    check(a, b, c, d, x, dtype)


def _switch_cases():
    """(dtype, c, T) for n = 1000: every CR level count the dtype's R_max allows
    and every T the reduced system has rows for (no collection-time skips)."""
    out = []
    for dtype in (np.float32, np.float64):
        for c_lv in (0, 1, 2, 3, 4):
            if dtype == np.float64 and c_lv > 3:  # R_max = 8 for fp64
                continue
            nred = -(-1000 // (1 << c_lv))
            threads = max(32, -(-nred // 32) * 32)
            for T in (1, 4, 32, 64, 1024):
                if T <= threads:
                    out.append((dtype, c_lv, T))
    return out


SWITCH_CASES = _switch_cases()


@pytest.mark.parametrize("dtype,c_lv,T", SWITCH_CASES)
def test_onchip_switch_points(tds, dtype, c_lv, T):
    """Every (c, T) switch point of the hybrid CR/PCR-Thomas kernel: c = 0 is the
    paper's PCR-Thomas; T = threads is pure PCR on the reduced system; T = 1 is
    a single Thomas chain."""
    n = 1000
    a, b, c, d = inputs.generate(n, 3, dtype, seed=5)
    x, _ = run(tds, a, b, c, d, params=dict(cr_levels=c_lv, thomas_chains=T))
    check(a, b, c, d, x, dtype)


# ------------------------------------------------ cluster (DSMEM) on-chip kernel

def _cluster_cases():
    """(dtype, n, C, T, c2) combinations the cluster kernel holds: the subsystem
    fits C CTAs of <= 512 threads and T <= the leader's reduced rows."""
    out = []
    for dtype in (np.float32, np.float64):
        c_lv = 4 if dtype == np.float32 else 3
        for n in (16384, 65536, 100003, 131072):
            for cl in (2, 4, 8, 16):
                nred = -(-n // ((1 << c_lv) * cl))
                threads = max(32, -(-nred // 32) * 32)
                if threads > 512:
                    continue
                for T in (1, 32, 512):
                    for tl in (0, 1, 3, 5):
                        if T <= (threads >> tl) * cl:
                            out.append((dtype, n, cl, T, tl))
    return out


CLUSTER_CASES = _cluster_cases()


@pytest.mark.parametrize("dtype,n,cl,T,tl", CLUSTER_CASES)
def test_onchip_cluster(tds, dtype, n, cl, T, tl):
    """One subsystem spread over a cluster of C CTAs (k = 0): CR in registers,
    reduced system gathered on the leader through DSMEM."""
    c_lv = 4 if dtype == np.float32 else 3
    a, b, c, d = inputs.generate(n, 3, dtype, seed=17)
    x, plan = run(tds, a, b, c, d, params=dict(k_pass=[], cr_levels=c_lv, thomas_chains=T, cluster=cl,
                                               tl_levels=tl))
    assert plan.info["cluster"] == cl and plan.info["k"] == 0
    check(a, b, c, d, x, dtype)


@pytest.mark.parametrize("dtype,n,cl", [(np.float32, 16384, 2), (np.float32, 16383, 2), (np.float32, 9001, 2),
                                        (np.float32, 8192, 1), (np.float32, 5000, 1), (np.float32, 1000, 1),
                                        (np.float32, 33, 1), (np.float64, 8192, 2), (np.float64, 6007, 2),
                                        (np.float64, 4096, 1), (np.float64, 777, 1), (np.float32, 65536, 8),
                                        (np.float32, 50001, 8), (np.float32, 32768, 4), (np.float32, 20000, 4),
                                        (np.float64, 32768, 8), (np.float64, 16000, 4)])
def test_onchip_k0_persistent(tds, dtype, n, cl):
    """k = 0 straight from a, b, c, d: the persistent TMA warp-form kernel on
    one CTA or a cluster of 2, 4 or 8 CTAs (DSMEM for the CTA boundaries, the
    top rows solved by one warp or by CTA 0 in shared memory), ragged sizes."""
    c_lv = 4 if dtype == np.float32 else 3
    a, b, c, d = inputs.generate(n, 5, dtype, seed=29)
    x, plan = run(tds, a, b, c, d, params=dict(k_pass=[], cr_levels=c_lv, thomas_chains=1, cluster=cl,
                                               tl_levels=5))
    assert plan.info["k"] == 0 and plan.info["cluster"] == cl
    check(a, b, c, d, x, dtype)


@pytest.mark.parametrize("n,tl,T", [(8192, 9, 1), (8192, 4, 32), (5000, 3, 8), (1000, 5, 1), (100, 5, 1)])
def test_onchip_thread_level_cr(tds, n, tl, T):
    """CR across threads inside one CTA (C = 1, c2 > 0) down to a tiny leader system."""
    a, b, c, d = inputs.generate(n, 4, np.float32, seed=23)
    R = 16 if n > 4096 else 4
    x, plan = run(tds, a, b, c, d, params=dict(k_pass=[], cr_levels=R.bit_length() - 1, thomas_chains=T,
                                               tl_levels=tl))
    check(a, b, c, d, x, np.float32)


@pytest.mark.parametrize("n,m,kp,cl", [(1 << 20, 2, [4], 8), (1 << 20, 1, [3], 16), (300001, 2, [2], 16),
                                       (1 << 19, 3, [1, 1], 16)])
def test_split_then_cluster(tds, n, m, kp, cl):
    a, b, c, d = inputs.generate(n, m, np.float32, seed=19)
    x, plan = run(tds, a, b, c, d, params=dict(k_pass=kp, cr_levels=4, thomas_chains=64, cluster=cl))
    check(a, b, c, d, x, np.float32)


# ------------------------------------------------ split passes + on-chip

SPLIT_CASES = [
    # dtype, n, m, k_pass, c, T, tile
    (np.float32, 4096, 3, [1], 1, 32, 1024),
    (np.float32, 4096, 3, [2], 2, 16, 256),
    (np.float32, 5000, 2, [3], 0, 32, 1024),
    (np.float32, 65536, 2, [3], 4, 64, 8192),
    (np.float32, 70001, 2, [4], 4, 64, 4096),
    (np.float32, 1 << 20, 2, [7], 4, 64, 8192),
    (np.float32, 1 << 18, 1, [9], 2, 32, 8192),
    (np.float32, 123457, 1, [5, 4], 2, 32, 2048),
    (np.float32, 1 << 16, 3, [3, 3, 3], 0, 64, 512),
    (np.float32, 1000, 2, [6, 4], 0, 1, 1024),   # 2^k > n: empty slots
    (np.float32, 37, 4, [2, 2, 1], 0, 1, 32),
    # fp64 (R_max = 8: on-chip subsystems of <= 4096 rows)
    (np.float64, 4096, 3, [1], 1, 32, 1024),
    (np.float64, 4096, 3, [2], 2, 16, 256),
    (np.float64, 5000, 2, [3], 0, 32, 1024),
    (np.float64, 65536, 2, [4], 3, 64, 4096),
    (np.float64, 70001, 2, [5], 3, 64, 4096),
    (np.float64, 1 << 20, 2, [8], 3, 64, 4096),
    (np.float64, 1 << 18, 1, [9], 2, 32, 4096),
    (np.float64, 123457, 1, [5, 4], 2, 32, 2048),
    (np.float64, 1 << 16, 3, [3, 3, 3], 0, 64, 512),
    (np.float64, 1000, 2, [6, 4], 0, 1, 1024),
    (np.float64, 37, 4, [2, 2, 1], 0, 1, 32),
]


def _split_params(n, kp, c_lv, T, tile):
    return dict(k_pass=kp, cr_levels=c_lv, thomas_chains=T, split_tile_rows=tile,
                split_threads=512 if tile >= 8192 else 256)


@pytest.mark.parametrize("dtype,n,m,kp,c_lv,T,tile", SPLIT_CASES)
def test_split_then_onchip(tds, dtype, n, m, kp, c_lv, T, tile):
    a, b, c, d = inputs.generate(n, m, dtype, seed=33)
    x, plan = run(tds, a, b, c, d, params=_split_params(n, kp, c_lv, T, tile))
    check(a, b, c, d, x, dtype)


@pytest.mark.parametrize("theta", [1, 4, 148, 10 ** 6])
def test_cooperative_segments(tds, theta):
    """Stage 1 (several CTAs per system, theta large) and stage 2 (one CTA per
    system, theta small) produce the same x bit-exactly."""
    n, m = 200000, 3
    a, b, c, d = inputs.generate(n, m, np.float32, seed=3)
    base = dict(k_pass=[5], cr_levels=4, thomas_chains=32, split_tile_rows=4096)
    x0, _ = run(tds, a, b, c, d, params=dict(base, theta=1))
    x1, plan = run(tds, a, b, c, d, params=dict(base, theta=theta))
    assert np.array_equal(x0, x1)
    check(a, b, c, d, x1, np.float32)


# ------------------------------------------------ the split stage itself

def split_gpu(tds, a, b, c, d, params):
    import torch
    m, n = d.shape
    dt = "float32" if d.dtype == np.float32 else "float64"
    plan = tds.Plan(n, m, dt, device=0)
    plan.set_params(**dict({"cluster": 1, "tl_levels": 0}, **params))
    oa, oc, od = tds.split_batched(plan, *to_dev(a, b, c, d))
    torch.cuda.synchronize()
    return oa.cpu().numpy(), oc.cpu().numpy(), od.cpu().numpy(), plan


@pytest.mark.parametrize("dtype", [np.float32, np.float64])
@pytest.mark.parametrize("n,kp", [(1000, [3]), (4096, [5]), (777, [2, 2]), (20000, [4, 3]), (300, [9])])
def test_split_vs_oracle_pcr(tds, dtype, n, kp):
    """Split coefficients vs the oracle's textbook PCR (fp64), normalised by b'
    and put in canonical order (tds_plan_permutation == oracle.permutation)."""
    a, b, c, d = inputs.generate(n, 2, dtype, seed=12)
    ga, gc, gd, plan = split_gpu(tds, a, b, c, d, dict(k_pass=kp, cr_levels=0, thomas_chains=1,
                                                      split_tile_rows=1024, split_threads=256))
    k = sum(kp)
    perm = plan.permutation()
    assert np.array_equal(perm, oracle.permutation(n, k))
    sa, sb, sc, sd = oracle.pcr_split(a, b, c, d, k)
    ref = [v[:, perm] / sb[:, perm] for v in (sa, sc, sd)]
    tol = 1e-5 if dtype == np.float32 else 1e-13
    for g, r in zip((ga, gc, gd), ref):
        assert np.abs(g - r).max() <= tol * max(1.0, np.abs(r).max())


@pytest.mark.parametrize("n,kp", [(300, [1]), (300, [4]), (1000, [5]), (4099, [3, 3])])
def test_split_exact_zeros(tds, n, kp):
    """a' = 0 at the first row and c' = 0 at the last row of every subsystem (bit-exact)."""
    a, b, c, d = inputs.generate(n, 2, np.float32, seed=1)
    ga, gc, gd, plan = split_gpu(tds, a, b, c, d, dict(k_pass=kp, cr_levels=0, thomas_chains=1,
                                                      split_tile_rows=1024, split_threads=256))
    k = sum(kp)
    step = 1 << k
    off = 0
    for r in range(min(step, n)):
        nr = -(-(n - r) // step)
        assert np.all(ga[:, off] == 0) and np.all(gc[:, off + nr - 1] == 0)
        off += nr


@pytest.mark.parametrize("dtype", [np.float32, np.float64])
@pytest.mark.parametrize("kp", [[1], [3], [7], [4, 3]])
def test_split_poisson_interior_exact(tds, dtype, kp):
    """On tridiag(-1,2,-1) every normalised level gives interior a' = c' = -1/2
    exactly (1 - 1/4 - 1/4 = 1/2, rcp(1/2) = 2): pins long strides bit-exactly."""
    n = 5000
    a, b, c, d = inputs.generate(n, 1, dtype, family="poisson")
    ga, gc, gd, plan = split_gpu(tds, a, b, c, d, dict(k_pass=kp, cr_levels=3, thomas_chains=1,
                                                      split_tile_rows=1024, split_threads=256))
    k = sum(kp)
    perm = plan.permutation()
    rows = perm  # original row of each canonical position
    interior = (rows >= (1 << k)) & (rows <= n - 1 - (1 << k))
    assert interior.sum() > n // 2
    assert np.all(ga[0, interior] == -0.5) and np.all(gc[0, interior] == -0.5)


def test_split_fused_equals_multipass_and_tiles(tds):
    """Halo exactness: k = 6 fused in one pass == 3 + 3 in two passes == other
    tile sizes, bit-exactly (same row update on the same operands)."""
    n = 50000
    a, b, c, d = inputs.generate(n, 2, np.float32, seed=4)
    base = dict(cr_levels=0, thomas_chains=1, split_threads=256)
    r1 = split_gpu(tds, a, b, c, d, dict(base, k_pass=[6], split_tile_rows=1024))
    r2 = split_gpu(tds, a, b, c, d, dict(base, k_pass=[3, 3], split_tile_rows=1024))
    r3 = split_gpu(tds, a, b, c, d, dict(base, k_pass=[6], split_tile_rows=4096, theta=1))
    r4 = split_gpu(tds, a, b, c, d, dict(base, k_pass=[2, 2, 2], split_tile_rows=64))
    for other in (r2, r3, r4):
        for u, v in zip(r1[:3], other[:3]):
            assert np.array_equal(u, v)


PIPE_THREADS = [dict(split_threads=512), dict(split_threads=256, split_tile_rows=4096)]


@pytest.mark.parametrize("dtype", [np.float32, np.float64])
@pytest.mark.parametrize("n,kp", [(200004, [5]), (200004, [6]), (131072, [7]), (200004, [8]),
                                  (3588 * 3 + 4, [8]), (200004, [3, 8]), (200004, [8, 2]), (300000, [2]),
                                  (7424 * 2 + 36, [7]), (100000, [4, 4])])
@pytest.mark.parametrize("geom", PIPE_THREADS, ids=["t512", "t256"])
def test_split_deep_pipe_vs_oracle(tds, dtype, n, kp, geom):
    """k_p <= 8 in one pass (persistent TMA split kernel: 4 levels on
    consecutive rows, k_p - 4 on residue classes mod 16; 256- and 512-thread
    tiles) vs the oracle's textbook PCR, on tiles with ragged tails."""
    a, b, c, d = inputs.generate(n, 2, dtype, seed=23)
    ga, gc, gd, plan = split_gpu(tds, a, b, c, d, dict(geom, k_pass=kp, split_only=1))
    k = sum(kp)
    perm = plan.permutation()
    sa, sb, sc, sd = oracle.pcr_split(a, b, c, d, k)
    ref = [v[:, perm] / sb[:, perm] for v in (sa, sc, sd)]
    tol = 1e-5 if dtype == np.float32 else 1e-13
    for g, r in zip((ga, gc, gd), ref):
        assert np.abs(g - r).max() <= tol * max(1.0, np.abs(r).max())


@pytest.mark.parametrize("n", [1 << 20, (1 << 20) + 12344, 4100])
@pytest.mark.parametrize("geom", PIPE_THREADS, ids=["t512", "t256"])
def test_split_deep_fused_equals_multipass(tds, n, geom):
    """Bit-exact: [8] == [4, 4] == [2, 2, 2, 2] and [7] == [4, 3] (the same
    normalised row update on the same operands, whatever the layout)."""
    a, b, c, d = inputs.generate(n, 2, np.float32, seed=5)
    base = dict(geom, split_only=1)
    r8 = split_gpu(tds, a, b, c, d, dict(base, k_pass=[8]))
    for other in ([4, 4], [2, 2, 2, 2], [5, 3]):
        ro = split_gpu(tds, a, b, c, d, dict(base, k_pass=other))
        for u, v in zip(r8[:3], ro[:3]):
            assert np.array_equal(u, v)
    r7 = split_gpu(tds, a, b, c, d, dict(base, k_pass=[7]))
    ro = split_gpu(tds, a, b, c, d, dict(base, k_pass=[4, 3]))
    for u, v in zip(r7[:3], ro[:3]):
        assert np.array_equal(u, v)


DEEP_CASES = [  # (dtype, n, k_pass): ragged n, subsystems that fill the pipe kernel (512 threads x 64 bytes)
    (np.float32, (1 << 20) - 4 * 777, [7]), (np.float32, (1 << 20) - 4 * 777, [8]),
    (np.float32, (1 << 19) - 4 * 777, [6]),
    (np.float64, (1 << 20) - 4 * 777, [8]), (np.float64, (1 << 19) - 4 * 777, [7]),
    (np.float64, (1 << 18) - 4 * 777, [6])]


def _deep_params(dtype, kp):
    return dict(k_pass=kp, cr_levels=4 if dtype == np.float32 else 3, thomas_chains=1, tl_levels=5, cluster=1)


@pytest.mark.parametrize("dtype,n,kp", DEEP_CASES)
def test_single_pass_deep_split_solve(tds, dtype, n, kp):
    """Whole solve with one deep split pass + the pipelined on-chip kernel."""
    a, b, c, d = inputs.generate(n, 3, dtype, seed=44)
    x, plan = run(tds, a, b, c, d, params=_deep_params(dtype, kp))
    assert plan.info["passes"] == 1
    check(a, b, c, d, x, dtype)


# ------------------------------------------------ layout, aliasing, isolation

def test_batch_isolation(tds):
    n, m = 30000, 4
    a, b, c, d = inputs.generate(n, m, np.float32, seed=8)
    x0, _ = run(tds, a, b, c, d, params=dict(k_pass=[3], cr_levels=4, thomas_chains=64))
    d2 = d.copy(); b2 = b.copy()
    d2[2] *= 1e6; b2[2] += 5
    x1, _ = run(tds, a, b2, c, d2, params=dict(k_pass=[3], cr_levels=4, thomas_chains=64))
    for s in (0, 1, 3):
        assert np.array_equal(x0[s], x1[s])


def test_inplace_and_stride(tds):
    import torch
    n, m, stride = 10000, 3, 10007
    a, b, c, d = inputs.generate(n, m, np.float32, seed=9)
    pad = lambda v: np.pad(v, ((0, 0), (0, stride - n)), constant_values=7.0)
    A, B, C, D = (pad(v).reshape(-1) for v in (a, b, c, d))
    plan = tds.Plan(n, m, "float32", device=0, batch_stride=stride)
    plan.set_params(k_pass=[2], cr_levels=4, thomas_chains=64)
    ta, tb, tc, td = to_dev(A, B, C, D)
    x = tds.solve_batched(plan, ta, tb, tc, td, out=td)  # in place
    torch.cuda.synchronize()
    xs = x.cpu().numpy().reshape(m, stride)
    assert np.all(xs[:, n:] == 7.0)  # padding untouched
    check(a, b, c, d, xs[:, :n], np.float32)


STRIDE_PLANS = [dict(k_pass=[], cr_levels=4, thomas_chains=16, cluster=2, tl_levels=5),   # k = 0 cluster kernel
                dict(k_pass=[2], cr_levels=4, thomas_chains=1, cluster=1, tl_levels=5),  # TMA split + pipe
                dict(k_pass=[7], cr_levels=2, thomas_chains=1, cluster=1, tl_levels=5),  # deep split, 4-D store
                dict(k_pass=[3, 2], cr_levels=4, thomas_chains=1, cluster=1, tl_levels=5)]


@pytest.mark.parametrize("plan_kw", STRIDE_PLANS, ids=["k0c2", "k2", "k7", "k3+2"])
@pytest.mark.parametrize("inplace", [False, True])
def test_tma_paths_stride_inplace(tds, plan_kw, inplace):
    """16-byte aligned batch stride > n (TMA tensor maps with a slot stride)
    in place and out of place: the padding between systems stays untouched."""
    import torch
    n, m, stride = 10000, 3, 10012
    a, b, c, d = inputs.generate(n, m, np.float32, seed=10)
    pad = lambda v: np.pad(v, ((0, 0), (0, stride - n)), constant_values=7.0)
    A, B, C, D = (pad(v).reshape(-1) for v in (a, b, c, d))
    plan = tds.Plan(n, m, "float32", device=0, batch_stride=stride)
    plan.set_params(**plan_kw)
    ta, tb, tc, td = to_dev(A, B, C, D)
    out = td if inplace else torch.full_like(td, 7.0)
    x = tds.solve_batched(plan, ta, tb, tc, td, out=out)
    torch.cuda.synchronize()
    xs = x.cpu().numpy().reshape(m, stride)
    assert np.all(xs[:, n:] == 7.0)
    check(a, b, c, d, xs[:, :n], np.float32)


def test_batch_isolation_k0_cluster(tds):
    """A poisoned neighbour system leaves the others bit-identical (k = 0 cluster kernel)."""
    n, m = 16000, 4
    a, b, c, d = inputs.generate(n, m, np.float32, seed=8)
    kw = dict(k_pass=[], cr_levels=4, thomas_chains=16, cluster=2, tl_levels=5)
    x0, _ = run(tds, a, b, c, d, params=kw)
    d2 = d.copy(); b2 = b.copy()
    d2[2] *= 1e6; b2[2] += 5
    x1, _ = run(tds, a, b2, c, d2, params=kw)
    for s in (0, 1, 3):
        assert np.array_equal(x0[s], x1[s])


def test_workspace_errors(tds):
    import torch
    n, m = 4096, 2
    a, b, c, d = inputs.generate(n, m, np.float32, seed=1)
    plan = tds.Plan(n, m, "float32", device=0)
    plan.set_params(k_pass=[2], cr_levels=2, thomas_chains=32)
    ta, tb, tc, td = to_dev(a, b, c, d)
    small = torch.empty(plan.workspace_bytes - 256, dtype=torch.uint8, device="cuda")
    with pytest.raises(tds.TdsError) as e:
        tds.solve_batched(plan, ta, tb, tc, td, workspace=small)
    assert e.value.name == "TDS_ERR_WORKSPACE"


# ------------------------------------------------ other value families (fp64, kappa-scaled)

@pytest.mark.parametrize("family,kw", [("poisson", {}), ("const", {"param": 0.01}), ("adi", {"param": 10.0}),
                                       ("weak", {"param": 0.1}), ("weak", {"param": 0.01})])
def test_families_fp64(tds, family, kw):
    n, m = 100000, 2
    a, b, c, d = inputs.generate(n, m, np.float64, seed=2, family=family, **kw)
    x, _ = run(tds, a, b, c, d, params=dict(k_pass=[5], cr_levels=3, thomas_chains=32))
    xr = oracle.thomas(a, b, c, d)
    assert oracle.backward_error(a, b, c, d, x) <= 1e-13
    if family == "poisson":
        kappa = 4 * (n + 1) ** 2 / math.pi ** 2
        assert oracle.rel_err(x, xr) <= 100 * kappa * 2.2e-16
    else:
        assert oracle.rel_err(x, xr) <= 1e-10


# ------------------------------------------------ BASELINE.json configs (bench launch configuration)

@pytest.mark.parametrize("dtype", [np.float32])
def test_config1_full(tds, dtype):
    a, b, c, d = inputs.generate(1024, 1, dtype, seed=inputs.config_seed(1, dtype))
    for mode in ("default", "static"):
        x, _ = run(tds, a, b, c, d, mode=mode)
        check(a, b, c, d, x, dtype)


@pytest.mark.parametrize("cfg,n,m,dtype", [(2, 65536, 256, np.float32), (3, 1 << 20, 16, np.float32),
                                            (3, 1 << 20, 16, np.float64)])
def test_config_full_static_and_default(tds, cfg, n, m, dtype):
    a, b, c, d = inputs.generate(n, m, dtype, seed=inputs.config_seed(cfg, dtype))
    xr = oracle.thomas(a, b, c, d)
    for mode in ("static", "default"):
        x, plan = run(tds, a, b, c, d, mode=mode)
        check(a, b, c, d, x, dtype, xr=xr)


def test_config4_sampled(tds):
    """4096 x 16384 fp32: the full batch on the GPU, 48 sampled systems through the oracle."""
    n, m = 16384, 4096
    a, b, c, d = inputs.generate(n, m, np.float32, seed=inputs.config_seed(4, np.float32))
    x, _ = run(tds, a, b, c, d, mode="static")
    rng = np.random.default_rng(0)
    idx = np.sort(np.concatenate([[0, m - 1], rng.choice(m, 46, replace=False)]))
    check(a[idx], b[idx], c[idx], d[idx], x[idx], np.float32)


BENCH_SHAPES = [  # the tuned plans bench.py times (profiles/r01h_bench_*), pinned explicitly
    (2, np.float32, dict(k_pass=[], cr_levels=4, thomas_chains=16, cluster=8, tl_levels=5)),
    (3, np.float32, dict(k_pass=[7], cr_levels=4, thomas_chains=16, cluster=1, tl_levels=5, split_threads=512,
                         split_tile_rows=8192)),
    (3, np.float64, dict(k_pass=[8], cr_levels=3, thomas_chains=16, cluster=1, tl_levels=5, split_threads=512,
                         split_tile_rows=4096)),
    (4, np.float32, dict(k_pass=[], cr_levels=4, thomas_chains=32, cluster=2, tl_levels=5))]


@pytest.mark.parametrize("how", ["pinned", "tuned"])
@pytest.mark.parametrize("cfg,dtype,params", BENCH_SHAPES, ids=["cfg2", "cfg3f32", "cfg3f64", "cfg4"])
def test_bench_launch_configuration_full_size(tds, tmp_path, how, cfg, dtype, params):
    """BASELINE.json configs 2-4 at full size in the launch configuration
    bench.py times: the plan the tuner picks on this device (as bench.py does)
    and the tuned shape recorded in profiles/, against the oracle (config 4:
    every system on the GPU, 64 sampled systems through the oracle)."""
    import torch
    n, m = {2: (65536, 256), 3: (1 << 20, 16), 4: (16384, 4096)}[cfg]
    a, b, c, d = inputs.generate(n, m, dtype, seed=inputs.config_seed(cfg, dtype))
    plan = tds.Plan(n, m, "float32" if dtype == np.float32 else "float64", device=0, mode="static")
    if how == "tuned":
        plan.tune(cache_path=str(tmp_path / "tune.txt"))
    else:
        plan.set_params(**params)
    ta, tb, tc, td = to_dev(a, b, c, d)
    x = tds.solve_batched(plan, ta, tb, tc, td)
    torch.cuda.synchronize()
    x = x.cpu().numpy()
    if cfg == 4:
        idx = np.sort(np.concatenate([[0, m - 1], np.random.default_rng(1).choice(m, 62, replace=False)]))
        a, b, c, d, x = a[idx], b[idx], c[idx], d[idx], x[idx]
    check(a, b, c, d, x, dtype)


@pytest.mark.slow
def test_config5_single_gpu_part(tds):
    """1 x 2^26 fp32 (the single-GPU half of config 5's schedule: 2 passes)."""
    n = 1 << 26
    a, b, c, d = inputs.generate(n, 1, np.float32, seed=5)
    x, plan = run(tds, a, b, c, d, mode="static")
    assert plan.info["passes"] == 2
    check(a, b, c, d, x, np.float32)


def test_tuner_runs_and_caches(tds, tmp_path):
    import torch
    n, m = 1 << 18, 8
    a, b, c, d = inputs.generate(n, m, np.float32, seed=1)
    plan = tds.Plan(n, m, "float32", device=0)
    cache = str(tmp_path / "tune.txt")
    trials = plan.tune(cache_path=cache)
    assert trials >= 3
    info = plan.info
    assert info["mode"] == 2 and info["tuned"] == 1
    ta, tb, tc, td = to_dev(a, b, c, d)
    x = tds.solve_batched(plan, ta, tb, tc, td)
    torch.cuda.synchronize()
    check(a, b, c, d, x.cpu().numpy(), np.float32)
    plan2 = tds.Plan(n, m, "float32", device=0)
    assert plan2.tune(cache_path=cache) == 0  # saved result reused
    assert plan2.info["k"] == info["k"] and plan2.info["thomas_chains"] == info["thomas_chains"]


@pytest.mark.parametrize("chunk", [1, 2, 3, 7])
def test_chunked_equals_unchunked(tds, chunk):
    """L2-resident chunks run the same kernels on each system: x bit-identical."""
    n, m = 100000, 7
    a, b, c, d = inputs.generate(n, m, np.float32, seed=29)
    base = dict(k_pass=[4, 2], cr_levels=4, thomas_chains=32, cluster=1, tl_levels=0)
    x0, _ = run(tds, a, b, c, d, params=dict(base, chunk_systems=0))
    x1, plan = run(tds, a, b, c, d, params=dict(base, chunk_systems=chunk))
    assert plan.info["chunks"] == -(-m // chunk)
    assert np.array_equal(x0, x1)
    check(a, b, c, d, x1, np.float32)
    g0 = split_gpu(tds, a, b, c, d, dict(base, chunk_systems=0))
    g1 = split_gpu(tds, a, b, c, d, dict(base, chunk_systems=chunk))
    for u, v in zip(g0[:3], g1[:3]):
        assert np.array_equal(u, v)


PIPE_PATH_SHAPES = {np.float32: [(1 << 20, [4, 3]), (777777, [3, 4]), (300000, [6]), (70000, [4])],
                    np.float64: [(1 << 20, [4, 4]), (777777, [4, 4]), (300000, [7]), (70000, [5])]}
PIPE_PATH_CASES = [(dt, n, kp, tl, T) for dt, shapes in PIPE_PATH_SHAPES.items() for n, kp in shapes
                   for tl, T in [(0, 64), (3, 32), (5, 1), (5, 4)]]


def _pipe_params(dtype, kp, tl, T):
    return dict(k_pass=kp, cr_levels=4 if dtype == np.float32 else 3, thomas_chains=T, tl_levels=tl, cluster=1)


@pytest.mark.parametrize("dtype,n,kp,tl,T", PIPE_PATH_CASES)
def test_onchip_pipe_paths(tds, dtype, n, kp, tl, T):
    """The persistent TMA-pipelined on-chip kernel (k > 0, cluster 1, 64 bytes
    of rows per thread), shared-memory and warp-shuffle (tl_levels = 5) forms."""
    a, b, c, d = inputs.generate(n, 2, dtype, seed=41)
    x, plan = run(tds, a, b, c, d, params=_pipe_params(dtype, kp, tl, T))
    check(a, b, c, d, x, dtype)


# ------------------------------------------- back-to-back solves on one stream

@pytest.mark.parametrize("dtype", [np.float32, np.float64])
def test_back_to_back_shared_workspace(tds, dtype):
    """Several solves of different plans enqueued back to back on one stream with
    no host synchronisation, all through ONE workspace buffer and some writing x
    over the previous solve's input: the programmatic-dependent-launch waits
    (griddepcontrol.wait before any global access) and the L2 discards of dead
    scratch lines must leave every result equal to its own solve run alone."""
    import torch
    dt = "float32" if dtype == np.float32 else "float64"
    cases = [(1 << 17, 4, {"k_pass": [5], "cr_levels": 4 if dtype == np.float32 else 3, "thomas_chains": 4,
                           "tl_levels": 5}),
             (65536, 6, {"k_pass": [4], "cr_levels": 3 if dtype == np.float32 else 2, "thomas_chains": 32,
                         "tl_levels": 0}),
             (8192, 8, None),                      # k = 0, static
             ((1 << 16) + 1000, 3, {"k_pass": [4, 2], "cr_levels": 2, "thomas_chains": 32, "tl_levels": 0})]
    plans, data, refs, wbytes = [], [], [], 0
    for i, (n, m, params) in enumerate(cases):
        a, b, c, d = inputs.generate(n, m, dtype, seed=40 + i)
        plan = tds.Plan(n, m, dt, device=0, mode="static")
        if params:
            plan.set_params(**dict({"cluster": 1}, **params))
        plans.append(plan)
        data.append(to_dev(a, b, c, d))
        refs.append((a, b, c, d))
        wbytes = max(wbytes, plan.workspace_bytes)
    ws = torch.empty(max(wbytes, 1), dtype=torch.uint8, device="cuda")
    outs = [torch.empty_like(dv[3]) for dv in data]
    torch.cuda.synchronize()
    for rep in range(3):
        for plan, (ta, tb, tc, td), x in zip(plans, data, outs):
            tds.solve_batched(plan, ta, tb, tc, td, out=x, workspace=ws)
    torch.cuda.synchronize()
    for (a, b, c, d), x in zip(refs, outs):
        check(a, b, c, d, x.cpu().numpy(), dtype)


@pytest.mark.parametrize("n", [8192 * 5 + 1, 8192 * 5 + 32])
def test_unaligned_slots_no_discard(tds, n):
    """Slots that are not whole 128-byte lines (ceil(n / 2^k) not a multiple of
    32 floats) disable the L2 discards; the result must not depend on it."""
    a, b, c, d = inputs.generate(n, 6, np.float32, seed=n)
    x, plan = run(tds, a, b, c, d, params={"k_pass": [3], "cr_levels": 4, "thomas_chains": 4, "tl_levels": 5})
    assert plan.info["slot_rows"] * 4 % 128 != 0
    check(a, b, c, d, x, np.float32)
    x2, _ = run(tds, a, b, c, d, params={"k_pass": [3], "cr_levels": 4, "thomas_chains": 4, "tl_levels": 5})
    assert np.array_equal(x, x2)


# ------------------------------- fused x placement (x_group: clusters of G CTAs)

XG_CASES = [  # (dtype, n, m, k_pass, G)
    (np.float32, 1 << 20, 3, [7], 8), (np.float32, 1 << 20, 2, [7], 4), (np.float32, 1 << 17, 5, [4], 8),
    (np.float32, 1 << 16, 3, [3], 8),           # 2^k == G: one group per system
    (np.float32, 1 << 15, 4, [2], 4),           # 2^k == G == 4
    (np.float32, 1 << 20, 2, [4, 3], 8),        # two split passes
    (np.float32, 24576, 3, [4], 8),             # 96 threads: 1536-row slots, 192-row segments (one box)
    (np.float32, 1 << 21, 1, [8], 8),           # 256 threads, m = 1
    (np.float64, 1 << 20, 2, [8], 2), (np.float64, 1 << 20, 2, [8], 4), (np.float64, 1 << 20, 2, [8], 8),
    (np.float64, 1 << 16, 3, [4], 4), (np.float64, 1 << 18, 2, [3, 3], 8)]


def _xg_params(dtype, kp, G):
    return dict(k_pass=kp, cr_levels=4 if dtype == np.float32 else 3, thomas_chains=1, tl_levels=5, x_group=G)


@pytest.mark.parametrize("dtype,n,m,kp,G", XG_CASES)
def test_fused_placement_vs_oracle_and_unfused(tds, dtype, n, m, kp, G):
    """x_group = G stores x straight from a cluster of G on-chip CTAs: the
    result is the oracle's within tolerance and BIT-identical to the same plan
    with the separate placement kernel (same arithmetic, different data path)."""
    a, b, c, d = inputs.generate(n, m, dtype, seed=60 + G)
    x, plan = run(tds, a, b, c, d, params=_xg_params(dtype, kp, G))
    assert plan.info["x_group"] == G and plan.info["launches"] == len(kp) + 1
    check(a, b, c, d, x, dtype)
    x0, _ = run(tds, a, b, c, d, params=_xg_params(dtype, kp, 0))
    assert np.array_equal(x, x0)


@pytest.mark.parametrize("inplace", [False, True])
@pytest.mark.parametrize("dtype", [np.float32, np.float64])
def test_fused_placement_stride_inplace(tds, inplace, dtype):
    """Padded 16-byte batch stride, in and out of place: the padding between
    systems is never written by the G-element TMA runs."""
    import torch
    n, m, stride = 1 << 17, 3, (1 << 17) + 16
    a, b, c, d = inputs.generate(n, m, dtype, seed=70)
    pad = lambda v: np.pad(v, ((0, 0), (0, stride - n)), constant_values=7.0)
    A, B, C, D = (pad(v).reshape(-1) for v in (a, b, c, d))
    dt = "float32" if dtype == np.float32 else "float64"
    plan = tds.Plan(n, m, dt, device=0, batch_stride=stride)
    plan.set_params(cluster=1, **_xg_params(dtype, [4] if dtype == np.float32 else [5], 8))
    ta, tb, tc, td = to_dev(A, B, C, D)
    out = td if inplace else torch.full_like(td, 7.0)
    x = tds.solve_batched(plan, ta, tb, tc, td, out=out)
    torch.cuda.synchronize()
    xs = x.cpu().numpy().reshape(m, stride)
    assert np.all(xs[:, n:] == 7.0)
    check(a, b, c, d, xs[:, :n], dtype)


def test_fused_placement_misaligned_x_falls_back(tds):
    """x not 16-byte aligned: the x_group plan runs the slot kernel + placement
    (same launch count) and gives the bit-identical result."""
    import torch
    n, m = 1 << 17, 2
    a, b, c, d = inputs.generate(n, m, np.float32, seed=71)
    x_ref, plan = run(tds, a, b, c, d, params=_xg_params(np.float32, [4], 8))
    ta, tb, tc, td = to_dev(a, b, c, d)
    buf = torch.zeros(m * n + 1, dtype=torch.float32, device="cuda")
    out = buf[1:].view(m, n)
    x = tds.solve_batched(plan, ta, tb, tc, td, out=out)
    torch.cuda.synchronize()
    assert np.array_equal(x.cpu().numpy(), x_ref)


def test_fused_placement_batch_isolation(tds):
    """A poisoned neighbour system leaves the others bit-identical (x_group = 8)."""
    n, m = 1 << 17, 4
    a, b, c, d = inputs.generate(n, m, np.float32, seed=72)
    kw = _xg_params(np.float32, [4], 8)
    x0, _ = run(tds, a, b, c, d, params=kw)
    d2 = d.copy(); b2 = b.copy()
    d2[2] *= 1e6; b2[2] += 5
    x1, _ = run(tds, a, b2, c, d2, params=kw)
    for s in (0, 1, 3):
        assert np.array_equal(x0[s], x1[s])


def test_fused_placement_back_to_back(tds):
    """Fused and unfused plans back to back on one stream through one workspace."""
    import torch
    cases = [(1 << 20, 2, _xg_params(np.float32, [7], 8)), (1 << 17, 3, _xg_params(np.float32, [4], 4)),
             (1 << 17, 3, _xg_params(np.float32, [4], 0)), (8192, 8, None)]
    plans, data, refs, wbytes = [], [], [], 0
    for i, (n, m, params) in enumerate(cases):
        a, b, c, d = inputs.generate(n, m, np.float32, seed=80 + i)
        plan = tds.Plan(n, m, "float32", device=0, mode="static")
        if params:
            plan.set_params(cluster=1, **params)
        plans.append(plan)
        data.append(to_dev(a, b, c, d))
        refs.append((a, b, c, d))
        wbytes = max(wbytes, plan.workspace_bytes)
    ws = torch.empty(max(wbytes, 1), dtype=torch.uint8, device="cuda")
    outs = [torch.empty_like(dv[3]) for dv in data]
    for rep in range(3):
        for plan, (ta, tb, tc, td), x in zip(plans, data, outs):
            tds.solve_batched(plan, ta, tb, tc, td, out=x, workspace=ws)
    torch.cuda.synchronize()
    for (a, b, c, d), x in zip(refs, outs):
        check(a, b, c, d, x.cpu().numpy(), np.float32)


# ------------------------------------------ batch-interleaved layout (tds_solve_interleaved)

IL_CASES = [  # (dtype, n, m, params or None for the static plan)
    (np.float32, 1024, 64, None), (np.float32, 1000, 33, None), (np.float32, 37, 5, None),
    (np.float32, 16384, 300, None),                                     # k = 0 cluster path
    (np.float32, 1 << 17, 7, dict(k_pass=[4], cr_levels=4, thomas_chains=16, tl_levels=5)),
    (np.float32, 300001, 3, None),                                      # ragged, split passes
    (np.float64, 4096, 129, None), (np.float64, 1 << 16, 9, dict(k_pass=[4], cr_levels=3, thomas_chains=16,
                                                                    tl_levels=5)),
    # whole 16-byte rows and columns: the TMA transposer (ragged edge tiles)
    (np.float32, 3000, 36, None), (np.float64, 4096, 130, None), (np.float64, 1000, 66, None),
    (np.float32, 1 << 17, 8, dict(k_pass=[4], cr_levels=4, thomas_chains=16, tl_levels=5))]


@pytest.mark.parametrize("dtype,n,m,params", IL_CASES)
@pytest.mark.parametrize("inplace", [False, True])
def test_interleaved_layout(tds, dtype, n, m, params, inplace):
    """Element i of system s at [i, s] of an (n, m) array: transposed in,
    solved by the plan's kernels, transposed back -- equal to the oracle on
    the same systems and BIT-identical to tds_solve_batched on the
    system-major copy (same kernels, same arithmetic)."""
    import torch
    a, b, c, d = inputs.generate(n, m, dtype, seed=90 + m)
    plan = tds.Plan(n, m, "float32" if dtype == np.float32 else "float64", device=0, mode="static")
    if params:
        plan.set_params(**dict({"cluster": 1}, **params))
    ti = [torch.from_numpy(np.ascontiguousarray(v.T)).cuda() for v in (a, b, c, d)]  # (n, m) interleaved
    out = ti[3] if inplace else None
    xi = tds.solve_interleaved(plan, *ti, out=out)
    ts = to_dev(a, b, c, d)
    xs = tds.solve_batched(plan, *ts)
    torch.cuda.synchronize()
    x = xi.cpu().numpy().T
    assert np.array_equal(x, xs.cpu().numpy())
    check(a, b, c, d, np.ascontiguousarray(x), dtype)


# ----------------------------------------------------------- CUDA graph capture

@pytest.mark.parametrize("params", [None, dict(k_pass=[7], cr_levels=4, thomas_chains=16, cluster=1, tl_levels=5),
                                    dict(k_pass=[], cr_levels=4, thomas_chains=16, cluster=2, tl_levels=5)],
                         ids=["static-k0", "k7-pipe", "k0-cluster2"])
def test_cuda_graph_capture_replay(tds, params):
    """A solve captured into a CUDA graph (all launches are stream-ordered,
    PDL edges included) replays to the bit-identical x of the eager call,
    with new inputs copied into the captured buffers between replays."""
    import torch
    n, m = (1 << 20, 2) if params and params["k_pass"] else (16384, 6)
    plan = tds.Plan(n, m, "float32", device=0, mode="static")
    if params:
        plan.set_params(**params)
    a, b, c, d = inputs.generate(n, m, np.float32, seed=101)
    ta, tb, tc, td = to_dev(a, b, c, d)
    x = torch.empty_like(td)
    ws = plan.workspace()
    s = torch.cuda.Stream()
    s.wait_stream(torch.cuda.current_stream())
    with torch.cuda.stream(s):
        tds.solve_batched(plan, ta, tb, tc, td, out=x, workspace=ws)  # warm-up (launch setup cached)
    torch.cuda.current_stream().wait_stream(s)
    torch.cuda.synchronize()
    g = torch.cuda.CUDAGraph()
    with torch.cuda.graph(g):
        tds.solve_batched(plan, ta, tb, tc, td, out=x, workspace=ws)
    for seed in (101, 102):
        a, b, c, d = inputs.generate(n, m, np.float32, seed=seed)
        for t, v in zip((ta, tb, tc, td), (a, b, c, d)):
            t.copy_(torch.from_numpy(v))
        x.zero_()
        g.replay()
        torch.cuda.synchronize()
        xg = x.cpu().numpy()
        xe = tds.solve_batched(plan, *to_dev(a, b, c, d)).cpu().numpy()
        assert np.array_equal(xg, xe)
        check(a, b, c, d, xg, np.float32)


# ------------------------------------------------ randomized plan fuzz (seeded)

def _fuzz_cases(count=320, seed=2024):
    rng = np.random.default_rng(seed)
    out = []
    for i in range(count):
        dtype = np.float32 if rng.random() < 0.7 else np.float64
        n = int(rng.choice([rng.integers(1, 5000), rng.integers(5000, 300000), 1 << int(rng.integers(10, 19))]))
        m = int(rng.integers(1, 7))
        k = int(rng.integers(0, 12))
        passes = 0 if k == 0 else int(rng.integers(1, min(3, k) + 1))
        kp = [] if k == 0 else [k // passes + (1 if j < k % passes else 0) for j in range(passes)]
        c_lv = int(rng.integers(0, 5 if dtype == np.float32 else 4))
        params = dict(k_pass=kp, cr_levels=c_lv, thomas_chains=int(2 ** rng.integers(0, 7)),
                      cluster=int(rng.choice([1, 1, 1, 2, 4, 8])), tl_levels=int(rng.choice([0, 1, 3, 5])),
                      x_group=int(rng.choice([0, 0, 0, 4, 8])), split_threads=int(rng.choice([256, 512])),
                      chunk_systems=int(rng.choice([0, 0, 1, 2])))
        out.append((i, dtype, n, m, params))
    try:  # keep the plans the planner accepts for B200 (host-only check; all of them if libtds is not built)
        import dataclasses
        import paper_conf_ipps_davidsonzo11_b200 as tds_mod
        from oracle import plan as rp
        props = dataclasses.asdict(rp.B200)
        keep = []
        for case in out:
            _, dt, n, m, params = case
            pl = tds_mod.Plan(n, m, "float32" if dt == np.float32 else "float64", props=props)
            try:
                pl.set_params(**dict({"cluster": 1, "tl_levels": 0}, **params))
                keep.append(case)
            except tds_mod.TdsError:
                pass
        return keep
    except (OSError, RuntimeError, ImportError):
        return out


@pytest.mark.parametrize("i,dtype,n,m,params", _fuzz_cases(), ids=lambda v: None)
def test_plan_fuzz(tds, i, dtype, n, m, params):
    """Seeded random plans (k, pass schedule, c, T, cluster, c2, x_group,
    split CTA size, chunking) over random n, m: every plan the planner accepts
    solves to the oracle's x within the tolerances."""
    a, b, c, d = inputs.generate(n, m, dtype, seed=1000 + i)
    x, plan = run(tds, a, b, c, d, params=params)  # the planner accepted it on CPU: it must run
    check(a, b, c, d, x, dtype)


# ------------------------------------- the paper's coalesced base-kernel variant (strided = 2)

CV_CASES = [  # (dtype, n, m, k, T): J = 1205 rows per subsystem fit in shared memory, the rest is global
    (np.float32, 16384, 7, 4, 16),        # L = 1024: every row on chip, no fallback
    (np.float32, 65536, 5, 3, 64),        # L = 8192: 85 % of the rows through the global fallback
    (np.float32, 100003, 3, 4, 64),       # ragged: residues of 6251 and 6250 rows in one group
    (np.float32, 8191 * 4 + 3, 2, 3, 1),  # T = 1: Thomas on whole subsystems, ragged
    (np.float32, 1 << 20, 2, 4, 128),     # L = 65536 (config-3 systems, one pass of 4 levels)
    (np.float32, 4096, 3, 4, 128),        # T = 128 of L = 256: chains of 2 rows
    (np.float32, 27, 3, 4, 2),            # n < 2^k: residues 27.. of the last group are empty
    (np.float32, 1205 * 8 + 8, 2, 3, 8),  # L = J + 1: exactly one global row per subsystem
    (np.float64, 32768, 3, 2, 64),        # fp64 group of 4 residues, L = 8192
    (np.float64, 9001, 4, 3, 256),        # fp64 ragged, T = 256 (1024 threads)
    (np.float64, 2411 * 4, 2, 2, 32)]     # fp64 L = 2411: J + 1206 global rows


def _cv_params(k, T):
    return dict(k_pass=[k], cr_levels=0, thomas_chains=T, cluster=1, tl_levels=0, strided=2)


def cv_stride(dtype, n):
    """The variant reads the TMA split's in-place output: systems start on 16 bytes."""
    e = 16 // np.dtype(dtype).itemsize
    return -(-n // e) * e


@pytest.mark.parametrize("dtype,n,m,k,T", CV_CASES)
def test_coalesced_variant(tds, dtype, n, m, k, T):
    """strided = 2: groups of 32 / sizeof(T) adjacent residues
    read as whole sectors, rows beyond shared memory read and written in the
    workspace (global fallback), PCR-Thomas, x stored in place: the oracle's
    x within the tolerances, two launches (ragged n on a 16-byte batch stride)."""
    import torch
    a, b, c, d = inputs.generate(n, m, dtype, seed=170 + k)
    stride = cv_stride(dtype, n)
    pad = lambda v: np.pad(v, ((0, 0), (0, stride - n)), constant_values=3.0)
    A, B, C, D = (torch.from_numpy(pad(v).reshape(-1)).cuda() for v in (a, b, c, d))
    plan = tds.Plan(n, m, "float32" if dtype == np.float32 else "float64", device=0, batch_stride=stride)
    plan.set_params(**_cv_params(k, T))
    assert plan.info["strided"] == 2 and plan.info["launches"] == 2
    out = torch.full_like(D, 5.0)
    tds.solve_batched(plan, A, B, C, D, out=out)
    torch.cuda.synchronize()
    xs = out.cpu().numpy().reshape(m, stride)
    assert np.all(xs[:, n:] == 5.0)
    check(a, b, c, d, np.ascontiguousarray(xs[:, :n]), dtype)


CV_BITEXACT = [  # (dtype, n, m, k, T): subsystems of <= 1024 rows, where the de-interleaved plan with the
    # same switch point (c = 0, c2 = 0, T, one CTA) runs the paper's PCR-Thomas base kernel (onchip.cu)
    (np.float32, 2048, 64, 3, 16), (np.float32, 16384, 9, 4, 64), (np.float32, 4000, 5, 3, 8),
    (np.float64, 4096, 6, 2, 32), (np.float64, 3002, 3, 3, 1)]


@pytest.mark.parametrize("dtype,n,m,k,T", CV_BITEXACT)
def test_coalesced_variant_bit_identical_to_deinterleaved(tds, dtype, n, m, k, T):
    """The coalesced variant changes only where the rows live (sector groups,
    global fallback), not the arithmetic: x is bit-identical to the
    de-interleaved path's PCR-Thomas base kernel under the same (k, T)."""
    a, b, c, d = inputs.generate(n, m, dtype, seed=182 + k)
    x2, p2 = run(tds, a, b, c, d, params=_cv_params(k, T))
    x0, p0 = run(tds, a, b, c, d, params=dict(_cv_params(k, T), strided=0))
    assert p0.info["onchip_form"] == p2.info["onchip_form"] == 0 and p0.info["launches"] == 3
    assert np.array_equal(x2, x0)
    check(a, b, c, d, x2, dtype)


@pytest.mark.parametrize("dtype,chunk", [(np.float32, 2), (np.float64, 3)])
def test_coalesced_variant_chunked(tds, dtype, chunk):
    """Chunked plans (chunk_systems): every chunk reuses the workspace (both
    buffers of the global fallback); x matches the unchunked plan bit for bit
    (same arithmetic per system) and the oracle."""
    n, m = 16384, 7
    a, b, c, d = inputs.generate(n, m, dtype, seed=181)
    x0, _ = run(tds, a, b, c, d, params=_cv_params(3, 64))
    x1, plan = run(tds, a, b, c, d, params=dict(_cv_params(3, 64), chunk_systems=chunk))
    assert plan.info["chunks"] == -(-m // chunk)
    assert np.array_equal(x0, x1)
    check(a, b, c, d, x1, dtype)


def test_coalesced_variant_stride_and_alignment(tds):
    """A padded batch stride leaves the padding; unaligned input rows are
    refused (UNSUPPORTED: the variant reads the TMA split's in-place output),
    and so is a batch stride that is not a 16-byte multiple (planner)."""
    import torch
    n, m, stride = 20000, 3, 20012
    a, b, c, d = inputs.generate(n, m, np.float32, seed=178)
    pad = lambda v: np.pad(v, ((0, 0), (0, stride - n)), constant_values=7.0)
    A, B, C, D = (torch.from_numpy(pad(v).reshape(-1)).cuda() for v in (a, b, c, d))
    plan = tds.Plan(n, m, "float32", device=0, batch_stride=stride)
    plan.set_params(**_cv_params(3, 32))
    out = torch.full_like(D, 7.0)
    tds.solve_batched(plan, A, B, C, D, out=out)
    torch.cuda.synchronize()
    xs = out.cpu().numpy().reshape(m, stride)
    assert np.all(xs[:, n:] == 7.0)
    check(a, b, c, d, xs[:, :n], np.float32)
    plan2 = tds.Plan(n, m, "float32", device=0)
    plan2.set_params(**_cv_params(3, 32))
    ta, tb, tc, td = (torch.zeros(m * n + 1, dtype=torch.float32, device="cuda")[1:].view(m, n) for _ in range(4))
    with pytest.raises(tds.TdsError) as e:
        tds.solve_batched(plan2, ta, tb, tc, td)
    assert e.value.name == "TDS_ERR_UNSUPPORTED"
    plan3 = tds.Plan(20001, m, "float32", device=0)
    with pytest.raises(tds.TdsError) as e:
        plan3.set_params(**_cv_params(3, 32))
    assert e.value.name == "TDS_ERR_UNSUPPORTED"


def test_coalesced_variant_interleaved_layout(tds):
    """The variant under the batch-interleaved entry point (tds_solve_interleaved)."""
    import torch
    n, m = 4096, 64
    a, b, c, d = inputs.generate(n, m, np.float32, seed=179)
    plan = tds.Plan(n, m, "float32", device=0)
    plan.set_params(**_cv_params(4, 16))
    ti = [torch.from_numpy(np.ascontiguousarray(v.T)).cuda() for v in (a, b, c, d)]
    x = tds.solve_interleaved(plan, *ti)
    torch.cuda.synchronize()
    check(a, b, c, d, x.cpu().numpy().T, np.float32)


# ------------------------------------- the paper's strided base-kernel variant

SV_CASES = [  # (dtype, n, m, k)
    (np.float32, 65536, 5, 3), (np.float32, 16384, 7, 1), (np.float32, 32768, 3, 2), (np.float32, 100003, 3, 4),
    (np.float32, 8191 * 4 + 3, 2, 2), (np.float64, 32768, 3, 3), (np.float64, 9001, 4, 2)]


@pytest.mark.parametrize("dtype,n,m,k", SV_CASES)
def test_strided_variant(tds, dtype, n, m, k):
    """strided = 1 (subsystems left interleaved by the split, gathered with
    stride 2^k on chip, x scattered in place): the oracle's x within the
    tolerances and BIT-identical to the de-interleaved path of the same plan
    (same split arithmetic, same on-chip solve)."""
    c_lv = 4 if dtype == np.float32 else 3
    kw = dict(k_pass=[k], cr_levels=c_lv, thomas_chains=1, tl_levels=5)
    a, b, c, d = inputs.generate(n, m, dtype, seed=70 + k)
    x1, plan = run(tds, a, b, c, d, params=dict(kw, strided=1))
    assert plan.info["strided"] == 1 and plan.info["launches"] == 2
    check(a, b, c, d, x1, dtype)
    x0, _ = run(tds, a, b, c, d, params=dict(kw, strided=0))
    assert np.array_equal(x1, x0)


def test_strided_variant_unaligned_input_and_stride(tds):
    """Unaligned input rows (no TMA split): the strided plan falls back to the
    de-interleaved kernels, same x; a padded batch stride leaves the padding."""
    import torch
    n, m = 20000, 3
    a, b, c, d = inputs.generate(n, m, np.float32, seed=77)
    kw = dict(k_pass=[2], cr_levels=4, thomas_chains=1, tl_levels=5, strided=1)
    xr, _ = run(tds, a, b, c, d, params=kw)
    plan = tds.Plan(n, m, "float32", device=0)
    plan.set_params(cluster=1, **kw)
    ta, tb, tc, td = (torch.zeros(m * n + 1, dtype=torch.float32, device="cuda")[1:].view(m, n) for _ in range(4))
    for t_, v in zip((ta, tb, tc, td), (a, b, c, d)):
        t_.copy_(torch.from_numpy(v))
    x = tds.solve_batched(plan, ta, tb, tc, td)
    torch.cuda.synchronize()
    assert np.array_equal(x.cpu().numpy(), xr)
    stride = n + 12
    pad = lambda v: np.pad(v, ((0, 0), (0, stride - n)), constant_values=7.0)
    A, B, C, D = (torch.from_numpy(pad(v).reshape(-1)).cuda() for v in (a, b, c, d))
    plan2 = tds.Plan(n, m, "float32", device=0, batch_stride=stride)
    plan2.set_params(cluster=1, **kw)
    out = torch.full_like(D, 7.0)
    tds.solve_batched(plan2, A, B, C, D, out=out)
    torch.cuda.synchronize()
    xs = out.cpu().numpy().reshape(m, stride)
    assert np.all(xs[:, n:] == 7.0)
    assert np.array_equal(xs[:, :n], xr)
