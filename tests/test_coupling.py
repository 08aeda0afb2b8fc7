"""Long-range coupling parity: every on-chip form of the CUDA path, on value
families whose solution couples rows far apart.

Why: on the diagonally dominant random
family (mu = 1) the normalised off-diagonals fall below 4e-8 after 4 PCR / CR
levels, so everything after the register / lane levels -- the cross-warp top
solve, the DSMEM hand-offs between the CTAs of a cluster, the all-gathered top
system, the leader's PCR-Thomas -- works on numerically diagonal systems and a
dropped or mis-indexed long-range term there is invisible.  Here the same
kernels solve, in fp64:

* Poisson tridiag(-1, 2, -1): every row couples to every row (closed-form
  condition number kappa_2 = sin^2(n pi / 2(n+1)) / sin^2(pi / 2(n+1)));
* tridiag(-1, 2 + 1e-6, -1): coupling length ~ 1/sqrt(1e-6) = 1000 rows;
* weak dominance (random, margin mu = 0.01);
* ADI diffusion a = c = -100, b = 201 (PAPER.md P:L50-53's application);

with tolerances 10 kappa eps_64 (Poisson, const) and 1e-10 (weak, ADI), and an
fp32 detector (tridiag(-1, 2 + delta, -1), delta = 1e-3 / 3e-4, n <= 16384,
coupling over 30-60 rows) at 10 kappa eps_32.  A debug build that drops one
long-range term per kernel (-DTDS_MUTATE=k, scripts/mutation_check.sh) fails
these tests (profiles/r02_mutation.md).

Each FORM names the kernel the C++ dispatch (csrc/api.cu solve_impl) selects
for its plan: k = 0 warp form -> onchip_cpipe (cluster 1/2/4/8), cluster 16 ->
onchip (generic, leader PCR-Thomas), k > 0 with 64 bytes of rows per thread ->
onchip_pipe (tl_levels 5: warp form, else shared-memory PCR-Thomas), x_group
-> onchip_gpipe, strided 1 -> onchip_strided, strided 2 -> onchip_coalesced,
k > 0 with cluster > 1 -> onchip.
Shapes are the BASELINE configs' (2^20 split by 2^8, 16384 on a cluster, 65536
on 16 CTAs) with enough systems that the persistent kernels loop.
"""
import math

import numpy as np
import pytest

import oracle
from paper_conf_ipps_davidsonzo11_b200 import inputs

F32, F64 = np.float32, np.float64
EPS = {F32: float(np.finfo(np.float32).eps), F64: float(np.finfo(np.float64).eps)}

_W = dict(thomas_chains=1, tl_levels=5)  # warp form: T is not used
# (id, dtype, n, m, params or None for the STATIC plan, api)
FORMS = [
    ("pipe_warp_k8", F64, 1 << 20, 2, dict(k_pass=[8], cr_levels=3, cluster=1, **_W), "batched"),
    ("pipe_smem_static", F64, 1 << 20, 2, None, "batched"),                      # k = 8, T = 64, tl = 0
    ("pipe_smem_tl3", F64, 1 << 20, 2, dict(k_pass=[8], cr_levels=3, thomas_chains=32, tl_levels=3, cluster=1),
     "batched"),
    ("pipe_warp_2pass", F64, 1 << 20, 2, dict(k_pass=[4, 4], cr_levels=3, cluster=1, **_W), "batched"),
    ("cpipe_c1", F64, 4096, 300, dict(k_pass=[], cr_levels=3, cluster=1, **_W), "batched"),
    ("cpipe_c2", F64, 8192, 200, dict(k_pass=[], cr_levels=3, cluster=2, **_W), "batched"),
    ("cpipe_c4", F64, 16384, 100, dict(k_pass=[], cr_levels=3, cluster=4, **_W), "batched"),
    ("cpipe_c8", F64, 32768, 40, dict(k_pass=[], cr_levels=3, cluster=8, **_W), "batched"),
    ("onchip_c16", F64, 65536, 3, dict(k_pass=[], cr_levels=3, thomas_chains=32, tl_levels=4, cluster=16),
     "batched"),
    ("split_cluster8", F64, 1 << 20, 2, dict(k_pass=[5], cr_levels=3, thomas_chains=32, tl_levels=3, cluster=8),
     "batched"),
    ("xgroup4", F64, 1 << 20, 2, dict(k_pass=[8], cr_levels=3, cluster=1, x_group=4, **_W), "batched"),
    ("xgroup8", F64, 1 << 20, 2, dict(k_pass=[8], cr_levels=3, cluster=1, x_group=8, **_W), "batched"),
    ("strided_k4", F64, 65536, 3, dict(k_pass=[4], cr_levels=3, cluster=1, strided=1, **_W), "batched"),
    ("interleaved_c4", F64, 16384, 40, dict(k_pass=[], cr_levels=3, cluster=4, **_W), "interleaved"),
    ("coalesced_k4", F64, 65536, 3, dict(k_pass=[4], cr_levels=0, thomas_chains=64, tl_levels=0, cluster=1,
                                         strided=2), "batched"),                   # 4096 rows: global fallback
    ("coalesced_k2_T8", F64, 4096, 8, dict(k_pass=[2], cr_levels=0, thomas_chains=8, tl_levels=0, cluster=1,
                                           strided=2), "batched"),                 # 1024 rows on chip
]

FAMILIES = [("poisson", {}), ("const", {"param": 1e-6}), ("weak", {"param": 0.01}), ("adi", {"param": 100.0})]

# fp32 detector: n <= 16384, coupling over ~30-100 rows
FORMS32 = [
    ("pipe_warp_k1", F32, 16384, 40, dict(k_pass=[1], cr_levels=4, cluster=1, **_W), "batched"),
    ("pipe_smem_static", F32, 16384, 40, None, "batched"),                       # k = 1, T = 64, tl = 0
    ("cpipe_c1", F32, 8192, 300, dict(k_pass=[], cr_levels=4, cluster=1, **_W), "batched"),
    ("cpipe_c2", F32, 16384, 200, dict(k_pass=[], cr_levels=4, cluster=2, **_W), "batched"),
    ("cpipe_c4", F32, 16384, 100, dict(k_pass=[], cr_levels=4, cluster=4, **_W), "batched"),
    ("cpipe_c8", F32, 16384, 60, dict(k_pass=[], cr_levels=4, cluster=8, **_W), "batched"),
    ("onchip_c16", F32, 16384, 4, dict(k_pass=[], cr_levels=3, thomas_chains=16, tl_levels=4, cluster=16),
     "batched"),
    ("xgroup8", F32, 16384, 40, dict(k_pass=[3], cr_levels=4, cluster=1, x_group=8, **_W), "batched"),
    ("strided_k1", F32, 16384, 40, dict(k_pass=[1], cr_levels=4, cluster=1, strided=1, **_W), "batched"),
    ("interleaved_c2", F32, 16384, 64, dict(k_pass=[], cr_levels=4, cluster=2, **_W), "interleaved"),
    ("coalesced_k3", F32, 16384, 40, dict(k_pass=[3], cr_levels=0, thomas_chains=16, tl_levels=0, cluster=1,
                                          strided=2), "batched"),                  # 2048 rows: global fallback
]


def const_kappa(n, delta):
    """2-norm condition number of tridiag(-1, 2 + delta, -1) (eigenvalues
    2 + delta - 2 cos(j pi / (n+1)))."""
    c = math.cos(math.pi / (n + 1))
    return (2 + delta + 2 * c) / (2 + delta - 2 * c)


def tolerance(family, kw, n, dtype):
    if family == "poisson":
        return 10 * const_kappa(n, 0.0) * EPS[dtype]
    if family == "const":
        return 10 * const_kappa(n, kw["param"]) * EPS[dtype]
    return 1e-10


@pytest.fixture(scope="module")
def tds():
    import torch
    assert torch.cuda.is_available()
    import paper_conf_ipps_davidsonzo11_b200 as m
    m._lib.load()
    return m


def solve(tds, a, b, c, d, params, api):
    import torch
    m, n = d.shape
    plan = tds.Plan(n, m, "float32" if d.dtype == np.float32 else "float64", device=0, mode="static")
    if params is not None:
        plan.set_params(**params)
    if api == "interleaved":
        ti = [torch.from_numpy(np.ascontiguousarray(v.T)).cuda() for v in (a, b, c, d)]
        x = tds.solve_interleaved(plan, *ti)
        torch.cuda.synchronize()
        return np.ascontiguousarray(x.cpu().numpy().T), plan
    ta, tb, tc, td = (torch.from_numpy(np.ascontiguousarray(v)).cuda() for v in (a, b, c, d))
    x = tds.solve_batched(plan, ta, tb, tc, td)
    torch.cuda.synchronize()
    return x.cpu().numpy(), plan


@pytest.mark.gpu
@pytest.mark.parametrize("family,kw", FAMILIES, ids=[f[0] for f in FAMILIES])
@pytest.mark.parametrize("form,dtype,n,m,params,api", FORMS, ids=[f[0] for f in FORMS])
def test_onchip_coupling_fp64(tds, form, dtype, n, m, params, api, family, kw):
    a, b, c, d = inputs.generate(n, m, dtype, seed=7, family=family, **kw)
    x, plan = solve(tds, a, b, c, d, params, api)
    if params is None:  # the STATIC plan is the paper's PCR-Thomas base kernel after one pass
        info = plan.info
        assert (info["k"], info["cluster"], info["tl_levels"], info["thomas_chains"]) == (8, 1, 0, 64)
    assert np.all(np.isfinite(x))
    xr = oracle.thomas(a, b, c, d)
    err = oracle.rel_err(x, xr)
    tol = tolerance(family, kw, n, dtype)
    assert err <= tol, f"{form}/{family}: rel_err {err:.3e} > {tol:.3e}"
    be = oracle.backward_error(a, b, c, d, x)
    assert be <= 1e-12, f"{form}/{family}: backward error {be:.3e}"


@pytest.mark.gpu
@pytest.mark.parametrize("delta", [1e-3, 3e-4])
@pytest.mark.parametrize("form,dtype,n,m,params,api", FORMS32, ids=[f[0] for f in FORMS32])
def test_onchip_coupling_fp32_detector(tds, form, dtype, n, m, params, api, delta):
    a, b, c, d = inputs.generate(n, m, dtype, seed=8, family="const", param=delta)
    x, plan = solve(tds, a, b, c, d, params, api)
    if params is None:
        info = plan.info
        assert (info["k"], info["cluster"], info["tl_levels"], info["thomas_chains"]) == (1, 1, 0, 64)
    assert np.all(np.isfinite(x))
    xr = oracle.thomas(a, b, c, d)
    err = oracle.rel_err(x, xr)
    # kappa of the fp32-rounded matrix (2 + delta rounds in fp32)
    tol = 10 * const_kappa(n, float(np.float32(2 + delta)) - 2) * EPS[F32]
    assert err <= tol, f"{form}/delta={delta}: rel_err {err:.3e} > {tol:.3e}"


# ---------------------------------------------------------------- CPU checks

def test_coupling_tolerances_are_tight():
    """The tolerances must leave a dropped coupling term visible: on the same
    families the solution changes by O(1) (relative) when the systems are cut
    in two halves (the effect of a lost long-range term), far above the
    tolerance."""
    for family, kw in FAMILIES[:2]:
        n = 16384
        a, b, c, d = inputs.generate(n, 1, F64, seed=7, family=family, **kw)
        x = oracle.thomas(a, b, c, d)
        a2, c2 = a.copy(), c.copy()
        a2[0, n // 2] = 0.0
        c2[0, n // 2 - 1] = 0.0
        xc = oracle.thomas(a2, b, c2, d)
        assert oracle.rel_err(xc, x) > 1e3 * tolerance(family, kw, n, F64)
    for delta in (1e-3, 3e-4):
        n = 16384
        a, b, c, d = inputs.generate(n, 1, F32, seed=8, family="const", param=delta)
        x = oracle.thomas(a, b, c, d)
        a2, c2 = a.copy(), c.copy()
        a2[0, n // 2 + 64] = 0.0  # a cut between two rows (a lost stride-1 coupling)
        c2[0, n // 2 + 63] = 0.0
        xc = oracle.thomas(a2, b, c2, d)
        tol = 10 * const_kappa(n, float(np.float32(2 + delta)) - 2) * EPS[F32]
        assert oracle.rel_err(xc, x) > 5 * tol


def test_const_kappa_closed_form():
    """const_kappa against the dense eigenvalues (numpy) on small n."""
    for n, delta in ((5, 0.0), (40, 1e-3), (64, 0.5)):
        A = np.diag(np.full(n, 2 + delta)) - np.diag(np.ones(n - 1), 1) - np.diag(np.ones(n - 1), -1)
        ev = np.linalg.eigvalsh(A)
        assert abs(const_kappa(n, delta) - ev.max() / ev.min()) <= 1e-9 * ev.max() / ev.min()
