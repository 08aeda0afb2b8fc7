"""CPU check that the GPU parity tests have no dead cases: every parameter set
the -m gpu tests pass to tds_plan_set_params is accepted by the planner for
B200 properties (tds_plan_from_props, no device needed).  The GPU tests call
the planner without try/except, so a rejected plan would fail there, never
skip silently."""
import dataclasses

import numpy as np
import pytest

from oracle import plan as rp

import test_coupling as tcp
import test_gpu_parity as tgp


@pytest.fixture(scope="module")
def tds():
    import paper_conf_ipps_davidsonzo11_b200 as m
    try:
        m._lib.load()
    except RuntimeError:
        import __graft_entry__
        __graft_entry__.build()
        m._lib.load()
    return m


def _accepts(tds, dtype, n, m, params, stride=0):
    p = tds.Plan(n, m, "float32" if dtype == np.float32 else "float64", props=dataclasses.asdict(rp.B200),
                 mode="static", batch_stride=stride)
    if params is not None:
        p.set_params(**params)
    return p.info


def _cases():
    out = []
    for dt, c_lv, T in tgp.SWITCH_CASES:
        out.append(("switch", dt, 1000, 3, dict(cluster=1, tl_levels=0, cr_levels=c_lv, thomas_chains=T)))
    for dt, n, cl, T, tl in tgp.CLUSTER_CASES:
        out.append(("cluster", dt, n, 3, dict(k_pass=[], cr_levels=4 if dt == np.float32 else 3, thomas_chains=T,
                                              cluster=cl, tl_levels=tl)))
    for dt, n, m, kp, c_lv, T, tile in tgp.SPLIT_CASES:
        out.append(("split", dt, n, m, dict(tgp._split_params(n, kp, c_lv, T, tile), cluster=1, tl_levels=0)))
    for dt, n, kp in tgp.DEEP_CASES:
        out.append(("deep", dt, n, 3, tgp._deep_params(dt, kp)))
    for dt, n, kp, tl, T in tgp.PIPE_PATH_CASES:
        out.append(("pipe", dt, n, 2, tgp._pipe_params(dt, kp, tl, T)))
    for fid, dt, n, m, params, api in tcp.FORMS + tcp.FORMS32:
        out.append(("coupling-" + fid, dt, n, m, params))
    for cfg, dt, params in tgp.BENCH_SHAPES:
        n, m = {2: (65536, 256), 3: (1 << 20, 16), 4: (16384, 4096)}[cfg]
        out.append((f"bench-cfg{cfg}", dt, n, m, params))
    for dt, n, m, kp, G in tgp.XG_CASES:
        out.append(("xgroup", dt, n, m, dict(tgp._xg_params(dt, kp, G), cluster=1)))
    return out


CV = [(dt, n, m, tgp._cv_params(k, T), tgp.cv_stride(dt, n)) for dt, n, m, k, T in tgp.CV_CASES] + \
    [(dt, 16384, 7, dict(tgp._cv_params(3, 64), chunk_systems=ch), 16384) for dt, ch in [(np.float32, 2),
                                                                                       (np.float64, 3)]] + \
    [(dt, n, m, p, 0) for dt, n, m, k, T in tgp.CV_BITEXACT for p in (tgp._cv_params(k, T),
                                                                    dict(tgp._cv_params(k, T), strided=0))]


@pytest.mark.parametrize("dtype,n,m,params,stride", CV)
def test_coalesced_case_is_accepted(tds, dtype, n, m, params, stride):
    assert _accepts(tds, dtype, n, m, params, stride)["strided"] == params["strided"]


CASES = _cases()


@pytest.mark.parametrize("kind,dtype,n,m,params", CASES, ids=[f"{c[0]}-{i}" for i, c in enumerate(CASES)])
def test_gpu_case_is_accepted(tds, kind, dtype, n, m, params):
    info = _accepts(tds, dtype, n, m, params)
    if params is not None and "k_pass" in params:
        assert info["k_pass"] == list(params["k_pass"])


def test_case_lists_are_not_empty():
    assert len(tgp.CLUSTER_CASES) > 100 and len(tgp.SWITCH_CASES) > 20
    assert len(tgp.PIPE_PATH_CASES) == 32 and len(tgp.DEEP_CASES) == 6
    assert sum(1 for c in tgp.SPLIT_CASES if c[0] == np.float64) == 11
