"""The self-tuner's search (§IV-D) on the CPU: tds_tune's
decoupled, seeded hill climb run through tds_tune_search with injected cost
functions instead of timed device solves (VERDICT r1 missing 4 / next 5).

Pinned here:
* decoupled stages make trials ADD, not multiply (the paper's
  16 + 32 = 48 instead of 16 x 32 = 512, tests/golden/paper_parameters.txt);
* the climb reaches the minimum of Fig. 5- and Fig. 6-shaped costs from the
  static seed and stops at a local minimum;
* candidates within 2 % do not replace the incumbent; the search is
  deterministic (reading R18);
* the cache round-trips ("save those results for future runs");
* the Thomas switch T is not searched in the warp form (it has no T);
* a cost that aborts (a device fault in tds_tune) fails with TDS_ERR_TUNE and
  leaves the plan unchanged.
"""
import dataclasses
import math
import os

import pytest

from oracle import plan as rp

GOLDEN = os.path.join(os.path.dirname(__file__), "golden")


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


def new_plan(tds, n=1 << 20, m=16, dtype="float32"):
    return tds.Plan(n, m, dtype, props=dataclasses.asdict(rp.B200), mode="static")


def run(tds, cost, **kw):
    p = new_plan(tds, **kw)
    seen = []

    def wrapped(q):
        seen.append(q)
        return cost(q)
    trials = p.tune_search(wrapped)
    assert trials == len(seen)
    return p, seen


def l2(v):
    return math.log2(max(v, 1))


# costs: 1 at the optimum, +0.5 per doubling / halving away from it
def cost_T(q):            # stage 3->4 switch only: optimum T = 8 (seed 64)
    return 1.0 + 0.5 * abs(l2(q["thomas_chains"]) - 3)


def cost_theta(q):        # stage 1->2 threshold only: optimum 8 x #SMs (seed #SMs)
    return 1.0 + 0.5 * abs(l2(q["theta"]) - l2(8 * 148))


def test_constant_cost_keeps_the_static_seed(tds):
    p0 = new_plan(tds).info
    p, seen = run(tds, lambda q: 1.0)
    i = p.info
    assert seen[0]["k_pass"] == p0["k_pass"] and seen[0]["thomas_chains"] == p0["thomas_chains"]
    assert (i["k"], i["k_pass"], i["thomas_chains"], i["theta"], i["cluster"]) == \
        (p0["k"], p0["k_pass"], p0["thomas_chains"], p0["theta"], p0["cluster"])
    assert i["mode"] == 2 and i["tuned"] == 1


def test_decoupled_trials_add_not_multiply(tds):
    """Two parameters of different stages (the Thomas switch T and the stage
    1->2 threshold theta), each with its optimum 3 doublings from the seed:
    the trials the search spends on both are the SUM of what it spends on
    each alone (the paper's 16 + 32 = 48, not 16 x 32 = 512)."""
    g = {}
    with open(os.path.join(GOLDEN, "paper_parameters.txt")) as f:
        for line in f:
            w = line.split("#")[0].split()
            if w:
                g[w[0]] = [int(v) for v in w[1:]]
    a, b, s, prod = g["decoupled_trials"]
    assert a + b == s and a * b == prod  # the paper's arithmetic, for the record
    _, s0 = run(tds, lambda q: 1.0)
    pT, sT = run(tds, cost_T)
    pV, sV = run(tds, cost_theta)
    pTV, sTV = run(tds, lambda q: cost_T(q) + cost_theta(q) - 1.0)
    dT, dV, dTV = len(sT) - len(s0), len(sV) - len(s0), len(sTV) - len(s0)
    assert dT > 0 and dV > 0
    assert dTV == dT + dV, (len(s0), dT, dV, dTV)
    assert dTV < dT * dV
    assert pT.info["thomas_chains"] == 8 and pV.info["theta"] == 8 * 148
    assert (pTV.info["thomas_chains"], pTV.info["theta"]) == (8, 8 * 148)


def fig6_cost(q):
    """Fig. 6 shape (time vs the Thomas switch): PCR work falls and
    Thomas latency grows with T -- a hyperbola a/T + b T, minimum at T = 128."""
    T = q["thomas_chains"]
    return 1.0 + 16.0 / T + T / 1024.0


def fig5_cost(q):
    """Fig. 5 shape (time vs the on-chip subsystem size): convex in
    k, minimum at k = 9 (n_sub = 2048), plus a per-pass cost."""
    return 1.0 + 0.3 * (q["k"] - 9) ** 2 + 0.2 * q["passes"]


def _neighbours_not_better(tds, p, cost):
    """Local minimum: no single-parameter step the search takes (T / 2, 2 T,
    k +- 1 with its schedule) is more than 2 % better."""
    best = cost(p.info)
    for key, vals in (("thomas_chains", (p.info["thomas_chains"] // 2, p.info["thomas_chains"] * 2)),):
        for v in vals:
            if v >= 1:
                q = dict(p.info, **{key: v})
                assert not cost(q) < 0.98 * best
    for dk in (-1, 1):
        k = p.info["k"] + dk
        for kpmax in (4, 8, 9):
            P = -(-k // kpmax)
            assert not cost(dict(p.info, k=k, passes=P)) < 0.98 * best


def test_climb_reaches_fig6_minimum(tds):
    p, seen = run(tds, fig6_cost)
    brute = min((2 ** j for j in range(0, 10)), key=lambda T: fig6_cost({"thomas_chains": T}))
    assert brute == 128
    assert p.info["thomas_chains"] == 128 and p.info["onchip_form"] == 0
    _neighbours_not_better(tds, p, fig6_cost)


def test_climb_reaches_fig5_minimum(tds):
    p, seen = run(tds, fig5_cost)
    assert p.info["k"] == 9 and p.info["passes"] == 1
    assert p.info["n_sub"] == (1 << 20) >> 9
    _neighbours_not_better(tds, p, fig5_cost)
    # both shapes at once: the decoupled search finds both minima
    p2, _ = run(tds, lambda q: fig5_cost(q) + fig6_cost(q) - 1.0)
    assert (p2.info["k"], p2.info["thomas_chains"]) in ((9, 128), (9, 64))  # T clamped by the new subsystem


def test_two_percent_tie_break_and_determinism(tds):
    """A neighbour 1 % faster does not replace the incumbent, 3 % faster does;
    two runs evaluate the same candidates in the same order."""
    def c(frac):
        return lambda q: frac if q["thomas_chains"] == 32 else 1.0
    p1, s1 = run(tds, c(0.99))
    assert p1.info["thomas_chains"] == 64
    p3, s3 = run(tds, c(0.97))
    assert p3.info["thomas_chains"] == 32
    p3b, s3b = run(tds, c(0.97))
    assert s3 == s3b and p3.info == p3b.info


def test_thomas_switch_not_searched_in_warp_form(tds):
    """The warp form (TDS_FORM_WARP_CR) has no Thomas switch: once the search
    is in it, no candidate differs from another only in T (T stays 1)."""
    def warp_fast(q):
        return 0.5 if q["tl_levels"] == 5 else 1.0
    p, seen = run(tds, warp_fast)
    assert p.info["onchip_form"] == 1 and p.info["thomas_chains"] == 1
    warp = [q for q in seen if q["tl_levels"] == 5 and q["cluster"] == 1]
    assert warp and all(q["thomas_chains"] == 1 for q in warp)


def test_cache_round_trip(tds, tmp_path):
    cache = str(tmp_path / "tune.txt")
    p = new_plan(tds)
    n1 = p.tune_search(fig6_cost, cache_path=cache)
    assert n1 > 0
    lines = open(cache).read().splitlines()
    assert len(lines) == 1 and "|n1048576|m16|" in lines[0]

    def never(q):
        raise AssertionError("a cache hit must not run trials")
    p2 = new_plan(tds)
    assert p2.tune_search(never, cache_path=cache) == 0
    assert p2.params_list() == p.params_list() and p2.info["tuned"] == 1
    p3 = new_plan(tds, m=8)  # another shape: a miss
    assert p3.tune_search(lambda q: 1.0, cache_path=cache) > 0
    assert len(open(cache).read().splitlines()) == 2


def test_aborting_cost_leaves_the_plan(tds):
    p = new_plan(tds)
    before = p.info
    with pytest.raises(tds.TdsError) as e:
        p.tune_search(lambda q: float("nan") if q["thomas_chains"] != 64 else 1.0)
    assert e.value.name == "TDS_ERR_TUNE"
    assert p.info == before
    with pytest.raises(tds.TdsError):
        p.tune_search(lambda q: 1e30)  # the seed refused
    assert p.info == before


def test_load_variants_are_a_tuner_dimension(tds):
    """The paper's two base-kernel load variants, chosen by the
    tuner per workload: when the coalesced variant with global
    fallback (strided = 2) is cheapest at the one-pass k <= 4 plans it is
    kept, and its Thomas switch T is then searched (its form is PCR-Thomas);
    when the strided gather is cheapest, that one is kept."""
    def coalesced_fast(q):
        if q["strided"] == 2:
            return 0.3 + 0.05 * abs(l2(q["thomas_chains"]) - 4)  # optimum T = 16
        return 1.0 if q["k"] <= 4 else 2.0
    p, seen = run(tds, coalesced_fast, n=65536, m=256)
    i = p.info
    assert i["strided"] == 2 and i["passes"] == 1 and i["k"] <= 4 and i["onchip_form"] == 0
    assert i["thomas_chains"] == 16 and i["cr_levels"] == 0 and i["tl_levels"] == 0
    assert {q["thomas_chains"] for q in seen if q["strided"] == 2} >= {64, 32, 16, 8}

    def strided_fast(q):  # the strided gather is a variant of the warp form (tl_levels = 5): reached through it
        if q["k"] > 4:
            return 2.0
        return 0.5 if q["strided"] == 1 else (0.9 if q["tl_levels"] == 5 and q["strided"] == 0 else 1.0)
    p1, seen1 = run(tds, strided_fast, n=65536, m=256)
    assert p1.info["strided"] == 1 and any(q["strided"] == 2 for q in seen1)
