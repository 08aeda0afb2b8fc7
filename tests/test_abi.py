"""C-ABI boundary tests that need no GPU: the library loads, exports every
symbol include/tds.h declares, the C++ planner matches the reference planner
bit-exactly, and argument errors are reported before anything is launched."""
import ctypes
import dataclasses
import os
import re

import numpy as np
import pytest

import oracle
from oracle import plan as rp

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


@pytest.fixture(scope="module")
def tds():
    lib_path = os.path.join(ROOT, "paper_conf_ipps_davidsonzo11_b200", "libtds.so")
    if not os.path.exists(lib_path):
        import __graft_entry__
        __graft_entry__.build()
    import paper_conf_ipps_davidsonzo11_b200 as m
    m._lib.load()
    return m


def header_functions():
    src = open(os.path.join(ROOT, "include", "tds.h")).read()
    src = re.sub(r"/\*.*?\*/", "", src, flags=re.S)
    return sorted(set(re.findall(r"\b(tds_[a-z_]+)\s*\(", src)))


def test_exports_every_header_symbol(tds):
    names = header_functions()
    assert len(names) >= 12
    lib = tds._lib.load()
    for name in names:
        assert hasattr(lib, name), name
    assert sorted(tds._lib.EXPORTED) == names
    assert tds.version() == 100


def test_status_strings(tds):
    lib = tds._lib.load()
    for code, name in tds._lib.STATUS_NAMES.items():
        assert lib.tds_status_string(code).decode().startswith(name)


def _props(p):
    return dataclasses.asdict(p)


CASES = []
for pname, props in [("B200", rp.B200)] + list(rp.TABLE_I.items()):
    for dtype in (rp.F32, rp.F64):
        for mode in (rp.DEFAULT, rp.STATIC):
            for n, m in [(1, 1), (2, 3), (255, 2), (256, 1), (257, 1), (1000, 7), (1024, 1), (4097, 3),
                         (65536, 256), (1 << 20, 16), (16384, 4096), (1 << 28, 1), (3 * 10 ** 6 + 7, 2),
                         (8192, 1), (8193, 5)]:
                CASES.append((pname, props, dtype, mode, n, m))


def _pow2ceil(v):
    p = 1
    while p < v:
        p *= 2
    return p


@pytest.mark.parametrize("pname,props,dtype,mode,n,m", CASES)
def test_planner_matches_reference(tds, pname, props, dtype, mode, n, m):
    """The method's integers (k, passes, k_pass, n_sub, number of subsystems,
    on-chip entry size, theta, T, segments) bit-exact vs the plain-Python
    reference planner (oracle/plan.py), which knows nothing of the kernels."""
    mname = "default" if mode == rp.DEFAULT else "static"
    dname = "float32" if dtype == rp.F32 else "float64"
    if pname != "B200":
        # Table I devices: the B200 kernels may not fit 16 / 48 KB of shared
        # memory; when the C++ planner accepts, the method's integers must agree.
        try:
            p = tds.Plan(n, m, dname, props=_props(props), mode=mname)
        except tds.TdsError as e:
            assert e.name == "TDS_ERR_UNSUPPORTED"
            return
    else:
        p = tds.Plan(n, m, dname, props=_props(props), mode=mname)
    got = p.info
    ref = rp.make_plan(props, dtype, n, m, mode, kp_max=got["split_kp_max"])
    if pname == "B200":
        assert got["split_kp_max"] == rp.KP_MAX[dtype]
    for f in ("k", "passes", "n_sub", "num_subsystems", "theta", "n_sub_target", "n_onchip_max"):
        assert got[f] == getattr(ref, f), (f, got[f], getattr(ref, f))
    assert got["k_pass"] == ref.k_pass[:ref.passes]
    # T: the mode's switch, unless the reduced on-chip system has fewer rows
    red = -(-got["n_sub"] // (1 << got["cr_levels"])) >> got["tl_levels"]
    assert got["thomas_chains"] == min(ref.thomas_switch, _pow2ceil(red))
    # segments: the rule's value, capped by the number of split tiles per system
    if ref.passes:
        tiles = -(-n // got["split_tile_eff"])
        assert got["split_segments"] == min(ref.segments, tiles)
    # build properties of the kernel shape (not the method's integers)
    assert got["cluster"] == 1 and got["chunk_systems"] == 0 and got["chunks"] == 1
    R = 1 << got["cr_levels"]
    assert R <= (16 if dtype == rp.F32 else 8)
    nt = got["onchip_threads"]
    assert nt % 32 == 0 and 32 <= nt <= props.max_threads_per_block
    assert nt >= -(-got["n_sub"] // R)
    assert got["launches"] == got["passes"] + 1 + (1 if got["k"] > 0 else 0)
    s = 4 if dtype == rp.F32 else 8
    if got["passes"]:
        # three normalised arrays of every row (x2 ping-pong for >= 2 passes)
        assert got["workspace_bytes"] >= (1 if got["passes"] == 1 else 2) * 3 * m * n * s
        assert got["slot_rows"] >= got["n_sub"] and (got["slot_rows"] * s) % 16 == 0
    else:
        assert got["workspace_bytes"] == 0


@pytest.mark.parametrize("n", [1, 5, 8, 100, 1023, 70000])
def test_permutation_matches_oracle(tds, n):
    for k in range(0, 9):
        p = tds.Plan(n, 1, props=_props(rp.B200), mode="static")
        if k:
            try:
                p.set_params(k_pass=[k], cr_levels=4 if n > 4096 else 0, thomas_chains=1)
            except tds.TdsError:
                continue
        assert np.array_equal(p.permutation(), oracle.permutation(n, p.info["k"]))


def test_plan_argument_errors(tds):
    lib = tds._lib.load()
    h = ctypes.c_void_p()
    props = tds._lib.DeviceProps(**_props(rp.B200))
    st = lambda *a: lib.tds_plan_from_props(ctypes.byref(h), ctypes.byref(props), *a)
    assert st(0, 0, 1, 0, 1) == 1          # n < 1
    assert st(0, 10, 0, 0, 1) == 1         # m < 1
    assert st(0, 10, 1, 5, 1) == 1         # stride < n
    assert st(2, 10, 1, 0, 1) == 1         # bad dtype
    assert st(0, 10, 1, 0, 2) == 1         # TUNED is set by tds_tune only
    assert st(0, 10, 1, 0, 9) == 1
    assert lib.tds_plan_from_props(None, ctypes.byref(props), 0, 10, 1, 0, 1) == 1
    assert st(0, 10, 1, 0, 1) == 0
    lib.tds_plan_destroy(h)


def test_set_params_validation(tds):
    p = tds.Plan(1 << 20, 4, props=_props(rp.B200))
    before = p.info
    with pytest.raises(tds.TdsError) as e:
        p.set_params(k_pass=[7], cr_levels=5)  # R = 32 > R_max
    assert e.value.name == "TDS_ERR_UNSUPPORTED"
    with pytest.raises(tds.TdsError):
        p.set_params(thomas_chains=48)  # not a power of two
    with pytest.raises(tds.TdsError):
        p.set_params(k_pass=[3], cr_levels=0)  # 131072-row subsystems do not fit on chip
    assert p.info == before  # unchanged after rejections
    p.set_params(k_pass=[5, 5], cr_levels=3, thomas_chains=16)
    i = p.info
    assert (i["k"], i["passes"], i["k_pass"], i["n_sub"], i["mode"]) == (10, 2, [5, 5], 1024, 2)
    slot = lambda kk: -(-(-(-(1 << 20) // (1 << kk))) // 4) * 4   # ceil(n / 2^kk) in 16-byte units
    assert i["workspace_bytes"] == 2 * 3 * 4 * max(4 * 32 * slot(5), 4 * 1024 * slot(10))


def test_solve_argument_errors_before_launch(tds):
    """Argument checks run on the host before any CUDA call; a plan built from
    fake properties has no device, so a valid call ends in DEVICE_MISMATCH or
    a CUDA error (no GPU here) -- never in a launch."""
    lib = tds._lib.load()
    p = tds.Plan(1000, 4, props=_props(rp.B200))
    p.set_params(k_pass=[2], cr_levels=0, thomas_chains=32)
    ws_need = p.workspace_bytes
    base = 1 << 40
    nbytes = 4 * 4000
    A, B, C, D, X = (base + i * (1 << 30) for i in range(5))
    W = base + 10 * (1 << 30)
    f = lambda *a: lib.tds_solve_batched(p.handle, *a, None)
    assert f(None, B, C, D, X, W, ws_need) == 1                 # NULL
    assert f(A + 2, B, C, D, X, W, ws_need) == 1                # misaligned
    assert f(A, B, C, D, A + 4, W, ws_need) == 1                # x overlaps a
    assert f(A, B, C, D, D + 8, W, ws_need) == 1                # x partially overlaps d
    assert f(A, B, C, D, X, None, ws_need) == 4                 # workspace NULL
    assert f(A, B, C, D, X, W, ws_need - 1) == 4                # too small
    assert f(A, B, C, D, X, W + 16, ws_need) == 4               # misaligned workspace
    assert f(A, B, C, D, X, A, ws_need) == 1                    # workspace overlaps an array
    assert f(A, B, C, D, D, W, ws_need) in (5, 7)               # valid (x == d): no device here
    assert nbytes < (1 << 30)


def test_x_group_validation(tds):
    """Fused x placement (x_group): accepted only where the gpipe kernel can
    store whole G-element runs of x (include/tds.h tds_params.x_group)."""
    p = tds.Plan(1 << 20, 16, props=_props(rp.B200))
    base = dict(k_pass=[7], cr_levels=4, thomas_chains=16, cluster=1, tl_levels=5)
    p.set_params(**base, x_group=8)
    i = p.info
    assert i["x_group"] == 8 and i["launches"] == 2  # split + on-chip, no placement kernel
    p.set_params(**base, x_group=0)
    assert p.info["launches"] == 3
    bad = [dict(x_group=3), dict(x_group=16), dict(x_group=2),          # fp32 runs need >= 4 elements
           dict(x_group=8, tl_levels=3), dict(x_group=8, cluster=2),
           dict(x_group=8, cr_levels=3),                                  # 32 bytes of rows per thread
           dict(x_group=8, k_pass=[], cr_levels=4)]                       # k = 0
    for kw in bad:
        with pytest.raises(tds.TdsError):
            p.set_params(**dict(base, **kw))
    q = tds.Plan((1 << 20) + 128, 2, props=_props(rp.B200))             # 2^7 does not divide n
    with pytest.raises(tds.TdsError):
        q.set_params(**base, x_group=8)
    q = tds.Plan(98304, 2, props=_props(rp.B200))                        # 768-row slots: 48 rows short of 64 x 16
    with pytest.raises(tds.TdsError):
        q.set_params(**dict(base, thomas_chains=1), x_group=8)
    r = tds.Plan(1 << 20, 2, "float64", props=_props(rp.B200))
    r.set_params(k_pass=[8], cr_levels=3, thomas_chains=16, cluster=1, tl_levels=5, x_group=2)
    assert r.info["launches"] == 2


def test_interleaved_workspace_and_errors(tds):
    """tds_interleaved_workspace_bytes: plan workspace + four 256-byte-rounded
    m x n copies; strided plans are refused; argument errors before launch."""
    p = tds.Plan(1 << 20, 16, props=_props(rp.B200))
    ws = p.info["workspace_bytes"]
    r256 = lambda v: -(-v // 256) * 256
    assert p.interleaved_workspace_bytes == r256(ws) + 4 * r256(16 * (1 << 20) * 4)
    q = tds.Plan(1000, 3, props=_props(rp.B200), batch_stride=1024)
    with pytest.raises(tds.TdsError) as e:
        q.interleaved_workspace_bytes
    assert e.value.name == "TDS_ERR_UNSUPPORTED"
    lib = tds._lib.load()
    h = p.handle
    assert lib.tds_solve_interleaved(h, None, 8, 8, 8, 8, 256, 1 << 40, None) == 1    # NULL a
    assert lib.tds_solve_interleaved(h, 8, 8, 8, 8, 8, None, 0, None) == 1            # x overlaps a
    assert lib.tds_solve_interleaved(h, 1 << 20, 2 << 30, 3 << 30, 4 << 30, 5 << 30, None, 0, None) == 4  # no ws
    assert lib.tds_interleaved_workspace_bytes(h, None) == 1


def test_strided_variant_validation(tds):
    """The paper's strided base-kernel variant (tds_params.strided): one split
    pass of <= 4 levels, warp form, cluster 1; two launches (no placement)."""
    p = tds.Plan(65536, 8, props=_props(rp.B200))
    base = dict(k_pass=[3], cr_levels=4, thomas_chains=16, cluster=1, tl_levels=5)
    p.set_params(**base, strided=1)
    assert p.info["strided"] == 1 and p.info["launches"] == 2
    for kw in [dict(strided=2), dict(strided=3), dict(strided=1, k_pass=[2, 1]), dict(strided=1, k_pass=[5]),
               dict(strided=1, tl_levels=3), dict(strided=1, cr_levels=3), dict(strided=1, cluster=2),
               dict(strided=1, x_group=8)]:
        with pytest.raises(tds.TdsError):
            p.set_params(**dict(base, **kw))


def test_coalesced_variant_validation(tds):
    """The paper's second base-kernel variant (tds_params.strided = 2,
    P:L286-292): one split pass of log2(32 / sizeof(T)) <= k <= 4 levels,
    cr_levels = tl_levels = 0, cluster 1; two launches (x stored in place),
    two workspace buffers (the global-fallback ping-pong), the PCR-Thomas
    form, and no on-chip size limit (rows beyond shared memory stay global)."""
    base = dict(k_pass=[3], cr_levels=0, thomas_chains=64, cluster=1, tl_levels=0, strided=2)
    p = tds.Plan(65536, 8, props=_props(rp.B200))
    p.set_params(**base)
    one = tds.Plan(65536, 8, props=_props(rp.B200))
    one.set_params(k_pass=[3], cr_levels=4, thomas_chains=1, cluster=1, tl_levels=5)
    assert p.info["strided"] == 2 and p.info["launches"] == 2
    assert p.info["workspace_bytes"] == 2 * one.info["workspace_bytes"]
    assert p.info["onchip_form"] == 0  # TDS_FORM_PCR_THOMAS
    assert p.info["onchip_threads"] == 512  # 8 residues x T = 64 chains
    big = tds.Plan(1 << 20, 16, props=_props(rp.B200))  # 65536-row subsystems: beyond any on-chip kernel
    big.set_params(**dict(base, k_pass=[4], thomas_chains=128))
    assert big.info["onchip_threads"] == 1024 and big.info["n_sub"] == 65536
    with pytest.raises(tds.TdsError):
        big.set_params(**dict(base, k_pass=[4], strided=0, cr_levels=4, tl_levels=5))
    d = tds.Plan(9001, 4, "float64", props=_props(rp.B200), batch_stride=9002)
    d.set_params(**dict(base, k_pass=[2], thomas_chains=256))  # fp64: G = 4, 4 x 256 threads
    assert d.info["onchip_threads"] == 1024
    for kw in [dict(k_pass=[2]), dict(k_pass=[5]), dict(k_pass=[2, 1]), dict(cr_levels=1), dict(tl_levels=1),
               dict(cluster=2), dict(x_group=8), dict(thomas_chains=256), dict(split_only=1)]:
        with pytest.raises(tds.TdsError):
            p.set_params(**dict(base, **kw))
