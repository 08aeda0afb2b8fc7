"""Reference planner (plain Python).  TEST INFRASTRUCTURE ONLY.

Writes out, step by step, the DEFAULT and STATIC parameter-selection rules of
DESIGN.md §"Planner (A1)" so the C++ planner in libtds can be checked against
it bit-exactly.  Shares no code with the C++ planner.

Paper sources:
* Workload decision "Enough Blocks?" -- Fig. 1.
* Default (machine-oblivious) parameters, §IV-B: on-chip entry at 256
  elements ("the weakest architecture only able to fit 256
  elements ... we select this as our switch point"), stage-1 stops at sixteen
  independent systems.
* Machine-query ("static") parameters, §IV-C: enter the on-chip kernel as soon
  as the subsystem fits in shared memory, switch to Thomas at 64
  independent subsystems per block (2x warp size), stage 1->2
  threshold from the processor count only.
* The default Thomas switch is unstated ("large enough that each warp has
  systems to solve"): reading R10 takes 32.
"""
from __future__ import annotations

import math
from dataclasses import dataclass, field

F32, F64 = 0, 1
DEFAULT, STATIC, TUNED = 0, 1, 2
MAX_PASSES = 8

# Paper constants (cited above)
DEFAULT_NSUB_TARGET = 256
DEFAULT_THETA = 16
STATIC_THOMAS_PER_WARP = 2     # 64 = 2 x warp size
DEFAULT_THOMAS = 32            # reading R10 (P:L602-607 gives no number)

# Build-side constants
DEFAULT_TILE = 1024
DEFAULT_SPLIT_THREADS = 256
DEFAULT_KP_MAX = 8
DEFAULT_G2_THREAD_CAP = 256
STATIC_SPLIT_THREADS = 512
SMEM_RESERVE = 1024            # per-CTA shared memory the runtime reserves


@dataclass
class Props:
    sm_count: int
    smem_optin_bytes: int
    smem_per_sm_bytes: int
    regs_per_sm: int
    max_threads_per_block: int
    warp_size: int
    cc_major: int
    cc_minor: int
    l2_bytes: int
    global_mem_bytes: int


# Table I as fake device properties; registers / threads from the
# CUDA programming guide's compute-capability tables (1.0, 1.3, 2.0).
TABLE_I = {
    "GeForce 8800 GTX": Props(14, 16384, 16384, 8192, 512, 32, 1, 0, 0, 768 << 20),
    "GeForce GTX 280": Props(30, 16384, 16384, 16384, 512, 32, 1, 3, 0, 1024 << 20),
    "GeForce GTX 470": Props(14, 49152, 49152, 32768, 1024, 32, 2, 0, 786432, 1280 << 20),
}
B200 = Props(148, 232448, 233472, 65536, 1024, 32, 10, 0, 132120576, 191 << 30)


def dsize(dtype: int) -> int:
    return 4 if dtype == F32 else 8


def cdiv(a: int, b: int) -> int:
    return -(-a // b)


def round_up(a: int, b: int) -> int:
    return cdiv(a, b) * b


def pow2ceil(x: int) -> int:
    p = 1
    while p < x:
        p *= 2
    return p


def static_cluster(props: Props) -> int:
    """Thread-block clusters exist from compute capability 9.0; 8 CTAs is the
    portable maximum.  Older devices (Table I) have none: 1."""
    return 8 if props.cc_major >= 9 else 1


def n_onchip_max(props: Props, dtype: int) -> int:
    """Largest power of two n whose four arrays fit in the shared memory of one
    cluster (4 n sizeof(T) <= (smem_optin - reserve) x C), capped at the
    on-chip kernel's register capacity (R_max x 512 threads x C)."""
    s = dsize(dtype)
    C = static_cluster(props)
    cap = r_max(dtype) * 512 * C
    budget = (props.smem_optin_bytes - SMEM_RESERVE) * C
    n = 1
    while n * 2 <= cap and 4 * (n * 2) * s <= budget:
        n *= 2
    return n


def r_max(dtype: int) -> int:
    return 16 if dtype == F32 else 8


REG_SPLIT_MAX_KP = 4          # split passes with k_p <= 4 use the register kernel
REG_SPLIT_TILE = 16 * 256 - 32  # rows it produces per CTA tile


@dataclass
class Plan:
    dtype: int
    mode: int
    n: int
    m: int
    batch_stride: int
    k: int = 0
    passes: int = 0
    k_pass: list = field(default_factory=lambda: [0] * MAX_PASSES)
    n_sub: int = 0
    num_subsystems: int = 0
    cr_levels: int = 0
    thomas_chains: int = 0
    onchip_threads: int = 0
    subsys_per_cta: int = 1
    cluster: int = 1
    tl_levels: int = 0
    chunk_systems: int = 0
    chunks: int = 1
    launches: int = 1
    split_tile_rows: int = 0
    split_threads: int = 0
    split_segments: int = 0
    theta: int = 0
    n_sub_target: int = 0
    n_onchip_max: int = 0
    split_kp_max: int = 0
    slot_rows: int = 0
    workspace_bytes: int = 0
    tuned: int = 0


def slot_rows(n: int, kk: int, dtype: int) -> int:
    """Workspace slot capacity of one subsystem after kk cumulative levels:
    ceil(n / 2^kk) rounded up to 16 bytes."""
    return round_up(cdiv(n, 1 << kk), 16 // dsize(dtype))


def split_smem_bytes(dtype: int, tile: int, kp: int) -> int:
    """Split-pass shared memory: 3 normalised arrays of the tile plus a
    (2^kp - 1)-row halo per side, padded by index >> max(kp, 5) against bank conflicts."""
    e = tile + 2 * ((1 << kp) - 1)
    return 3 * (e + (e >> max(kp, 5)) + 1) * dsize(dtype)


def segments(m_in: int, tiles: int, theta: int) -> int:
    """Stage 1 (cooperative, several CTAs per system) until theta independent
    systems exist, else Stage 2 (one CTA per system) -- Fig. 1 P:L169-187."""
    if m_in >= theta:
        return 1
    return max(1, min(tiles, cdiv(theta, m_in)))


def make_plan(props: Props, dtype: int, n: int, m: int, batch_stride: int = 0,
              mode: int = STATIC) -> Plan:
    if n < 1 or m < 1:
        raise ValueError("n, m >= 1")
    if batch_stride == 0:
        batch_stride = n
    if batch_stride < n:
        raise ValueError("batch_stride >= n")
    if mode not in (DEFAULT, STATIC):
        raise ValueError("mode")
    s = dsize(dtype)
    p = Plan(dtype=dtype, mode=mode, n=n, m=m, batch_stride=batch_stride)
    p.n_onchip_max = n_onchip_max(props, dtype)
    if mode == DEFAULT:
        target, T, theta = DEFAULT_NSUB_TARGET, DEFAULT_THOMAS, DEFAULT_THETA
        tile, g1t, kpmax, g2cap = DEFAULT_TILE, DEFAULT_SPLIT_THREADS, DEFAULT_KP_MAX, DEFAULT_G2_THREAD_CAP
        cmax = 1
    else:
        target = p.n_onchip_max
        T = STATIC_THOMAS_PER_WARP * props.warp_size
        theta = 32 * props.sm_count  # from the processor count
        tile = min(p.n_onchip_max, r_max(dtype) * 512)
        g1t = STATIC_SPLIT_THREADS
        cmax = static_cluster(props)
        kpmax = 9 if dtype == F32 else 8
        budget = props.smem_optin_bytes - SMEM_RESERVE
        while kpmax > 1 and (split_smem_bytes(dtype, tile, kpmax) > budget
                             or (1 << kpmax) > tile):
            kpmax -= 1
        g2cap = props.max_threads_per_block // 2
    p.n_sub_target, p.theta, p.split_tile_rows, p.split_threads, p.split_kp_max = target, theta, tile, g1t, kpmax

    # Stage 2->3 switch: split until each subsystem fits (k levels, 2^k subsystems).
    k = 0
    while cdiv(n, 1 << k) > target:
        k += 1
    p.k = k
    p.n_sub = cdiv(n, 1 << k)
    p.num_subsystems = m * min(1 << k, n)
    P = cdiv(k, kpmax) if k > 0 else 0
    if P > MAX_PASSES:
        raise ValueError("too many passes")
    p.passes = P
    if P:
        base, extra = divmod(k, P)
        for i in range(P):
            p.k_pass[i] = base + (1 if i < extra else 0)

    # Stage 3->4 switch inside the on-chip kernel: the smallest cluster of C
    # CTAs that holds the subsystem, R = 2^c rows per thread (c CR levels),
    # then PCR on the reduced system until T Thomas chains.
    C = 1
    while C < cmax and p.n_sub > C * r_max(dtype) * g2cap:
        C *= 2
    R = 1
    while cdiv(p.n_sub, R * C) > g2cap and R < r_max(dtype):
        R *= 2
    if C > 1 and R < 8:
        R = 8
    nred = cdiv(p.n_sub, R * C)
    p.cluster = C
    p.cr_levels = R.bit_length() - 1
    p.onchip_threads = max(32, round_up(nred, 32))
    # CR across threads until the leader's system has one row per thread
    p.tl_levels = C.bit_length() - 1
    p.thomas_chains = min(T, pow2ceil(cdiv(p.n_sub, R) >> p.tl_levels))

    # Kernel limits (the C++ planner rejects these plans as UNSUPPORTED).
    budget = props.smem_optin_bytes - SMEM_RESERVE
    for i in range(P):
        if p.k_pass[i] > REG_SPLIT_MAX_KP and split_smem_bytes(dtype, tile, p.k_pass[i]) > budget:
            raise ValueError("unsupported: split tile + halo exceeds shared memory")
    nt = p.onchip_threads
    if (3 * C * (nt >> p.tl_levels) + 4 * nt + 6 * (nt // 32) + 48) * s > budget:
        raise ValueError("unsupported: on-chip shared memory")

    # L2-resident chunking is a tuner dimension only (both planners seed 0).
    p.chunk_systems = 0
    mc = m
    p.chunks = cdiv(m, mc)
    p.launches = p.chunks * (P + 1 + (1 if k > 0 else 0))

    # Workspace: split output (normalised a, c, d) of one chunk in fixed slots; ping-pong if P >= 2.
    if P:
        kk, elems = 0, 0
        for i in range(P):
            kk += p.k_pass[i]
            elems = max(elems, mc * (1 << kk) * slot_rows(n, kk, dtype))
        E = round_up(elems, 64)
        p.slot_rows = slot_rows(n, k, dtype)
        p.workspace_bytes = (1 if P == 1 else 2) * 3 * E * s
        tile_eff = REG_SPLIT_TILE if p.k_pass[0] <= REG_SPLIT_MAX_KP else tile
        p.split_segments = segments(mc, cdiv(n, tile_eff), theta)
    return p
