"""Host-side checks of the split kernel's shared-memory transpose layout
(csrc/split_reg.cuh, tr34_phys / tr34_read; used by the fp32 512-thread
split tiles of csrc/split_pipe.cu).  Build properties of the kernel's index
arithmetic, not numerics: every layout-A store lands on its own word, every
layout-B load of a member inside the window reads the word that member was
stored to, no access leaves the buffer, and both directions are free of
shared-memory bank conflicts.  The constants are read from the header so the
test follows the kernel."""
import collections
import os
import re

import pytest

HDR = os.path.join(os.path.dirname(os.path.dirname(os.path.abspath(__file__))),
                   "paper_conf_ipps_davidsonzo11_b200", "csrc", "split_reg.cuh")

AV = 480          # valid A-blocks (members per class) of a 512-thread tile: 30 lanes x 16 warps
NWARPS = 16


def _const(name):
    m = re.search(r"constexpr int %s = (\d+);" % name, open(HDR).read())
    assert m, name
    return int(m.group(1))


W, C = _const("kTr34W"), _const("kTr34C")
SLACK = 32        # spare words after the three arrays (split_pipe.cu tbuf_elems)


def phys(m):      # tr34_phys
    return (m & 15) * W + (m >> 4)


def read_addr(rho, b, u, left):   # tr34_read: p = row + b - 1, member mb + u
    return rho * C + b - 1 + ((left + u) & 15) * W + ((left + u) >> 4)


def wavefronts(addrs):
    banks = collections.defaultdict(set)
    for a in addrs:
        banks[a % 32].add(a)
    return max(len(s) for s in banks.values())


def test_class_stride_holds_a_class():
    assert max(phys(m) for m in range(AV)) < C <= 16 * W


@pytest.mark.parametrize("left", [4, 8, 16])   # k_p = 5, 6 -> 4; 7 -> 8; 8 -> 16 (split_pipe.cu LEFT)
def test_reads_match_writes_and_stay_in_buffer(left):
    stored = {}
    for rho in range(16):
        for m in range(AV):
            a = rho * C + phys(m)
            assert a not in stored
            stored[a] = (rho, m)
    size = 16 * C
    for arr in range(3):
        for rho in range(16):
            for b in range(32):
                for u in range(16):
                    a = read_addr(rho, b, u, left)
                    assert 0 <= arr * size + a < 3 * size + SLACK
                    member = left - 16 + 16 * b + u
                    if 0 <= member < AV:
                        assert stored[a] == (rho, member)


def test_layout_a_stores_conflict_free():
    # warp w stores members 30 w + l - 1 (lanes 1..30), one class per instruction
    for w in range(NWARPS):
        assert wavefronts([phys(30 * w + lane - 1) for lane in range(1, 31)]) == 1


@pytest.mark.parametrize("left", [4, 8, 16])
def test_layout_b_loads_conflict_free(left):
    # one class per warp (lanes b = 0..31), member u of every lane per load
    for rho in range(16):
        for u in range(16):
            assert wavefronts([read_addr(rho, b, u, left) for b in range(32)]) == 1


def test_old_swizzle_had_store_conflicts():
    # the [rho][m] chunk swizzle this layout replaced: ~1.6 wavefronts per store
    def old(m):
        return (((m >> 2) ^ ((m >> 5) & 3)) << 2) | (m & 3)
    mean = sum(wavefronts([old(30 * w + lane - 1) for lane in range(1, 31)]) for w in range(NWARPS)) / NWARPS
    assert mean > 1.5
