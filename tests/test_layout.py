"""Host-side checks of the split kernel's shared-memory transpose layout
(csrc/split_reg.cuh, Tr34 / tr34_phys / tr34_read; used by the fp32
512-thread and fp64 256-thread split tiles of csrc/split_pipe.cu).  Build
properties of the kernel's index arithmetic, not numerics: every layout-A
store lands on its own element, every layout-B load of a member inside the
window reads the element that member was stored to, no access leaves the
buffer, and both directions are free of shared-memory bank conflicts.  The
constants are checked against the header."""
import collections
import os
import re

import pytest

HDR = os.path.join(os.path.dirname(os.path.dirname(os.path.abspath(__file__))),
                   "paper_conf_ipps_davidsonzo11_b200", "csrc", "split_reg.cuh")

# (element size, AV members per class, lanes per class chain, store groups of lanes that
# one shared-memory wavefront serves, bank units per wavefront)
SHAPES = {
    "f32": dict(W=34, C=540, SLACK=32, AV=480, CH=32, groups=[range(1, 31)], banks=32),
    # 8-byte stores: one wavefront per half-warp (lanes 1..15, 16..30 store; 16 bank pairs)
    "f64": dict(W=17, C=271, SLACK=0, AV=240, CH=16, groups=[range(1, 16), range(16, 31)], banks=16),
}
NWARPS = {"f32": 16, "f64": 8}


def test_header_constants():
    src = open(HDR).read()
    assert re.search(r"W = sizeof\(T\) == 4 \? 34 : 17;", src)
    assert re.search(r"C = sizeof\(T\) == 4 \? 540 : 271;", src)
    assert re.search(r"SLACK = sizeof\(T\) == 4 \? 32 : 0;", src)


def phys(m, W):      # tr34_phys
    return (m & 15) * W + (m >> 4)


def read_addr(rho, b, u, left, W, C):   # tr34_read: p = row + b - 1, member mb + u
    return rho * C + b - 1 + ((left + u) & 15) * W + ((left + u) >> 4)


def wavefronts(addrs, banks):
    by_bank = collections.defaultdict(set)
    for a in addrs:
        by_bank[a % banks].add(a)
    return max(len(s) for s in by_bank.values())


@pytest.mark.parametrize("dt", ["f32", "f64"])
def test_class_stride_holds_a_class(dt):
    g = SHAPES[dt]
    assert max(phys(m, g["W"]) for m in range(g["AV"])) < g["C"] <= 16 * g["W"]


@pytest.mark.parametrize("dt", ["f32", "f64"])
@pytest.mark.parametrize("left", [4, 8, 16])   # k_p = 5, 6 -> 4; 7 -> 8; 8 -> 16 (split_pipe.cu LEFT)
def test_reads_match_writes_and_stay_in_buffer(dt, left):
    g = SHAPES[dt]
    W, C, AV = g["W"], g["C"], g["AV"]
    stored = {}
    for rho in range(16):
        for m in range(AV):
            a = rho * C + phys(m, W)
            assert a not in stored
            stored[a] = (rho, m)
    size = 16 * C
    for arr in range(3):
        for rho in range(16):
            for b in range(g["CH"]):
                for u in range(16):
                    a = read_addr(rho, b, u, left, W, C)
                    assert 0 <= arr * size + a < 3 * size + g["SLACK"]
                    member = left - 16 + 16 * b + u
                    if 0 <= member < AV:
                        assert stored[a] == (rho, member)


@pytest.mark.parametrize("dt", ["f32", "f64"])
def test_layout_a_stores_conflict_free(dt):
    # warp w stores members 30 w + l - 1 (lanes 1..30), one class per instruction
    g = SHAPES[dt]
    for w in range(NWARPS[dt]):
        for lanes in g["groups"]:
            assert wavefronts([phys(30 * w + lane - 1, g["W"]) for lane in lanes], g["banks"]) == 1


@pytest.mark.parametrize("dt", ["f32", "f64"])
@pytest.mark.parametrize("left", [4, 8, 16])
def test_layout_b_loads_conflict_free(dt, left):
    # one class per chain of CH lanes (f32: a warp; f64: a half-warp), member u of every lane per load
    g = SHAPES[dt]
    for rho in range(16):
        for u in range(16):
            addrs = [read_addr(rho, b, u, left, g["W"], g["C"]) for b in range(g["CH"])]
            assert wavefronts(addrs, g["banks"]) == 1


def test_old_swizzle_had_store_conflicts():
    # the [rho][m] chunk swizzle this layout replaced: ~1.6 wavefronts per store
    def old(m):
        return (((m >> 2) ^ ((m >> 5) & 3)) << 2) | (m & 3)
    mean = sum(wavefronts([old(30 * w + lane - 1) for lane in range(1, 31)], 32) for w in range(16)) / 16
    assert mean > 1.5
