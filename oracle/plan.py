"""Reference planner (plain Python).  TEST INFRASTRUCTURE ONLY.

Writes out the paper's DEFAULT and machine-query ("static") parameter
selection -- the METHOD's integers only -- so the C++ planner in libtds can be
checked against it.  It knows nothing about the B200 kernels (CTA sizes, CR
levels in registers, clusters, workspace layout, split tiles): those are build
choices and are tested as properties of the C++ plan, not pinned here.  It
shares no code with the C++ planner.

Paper sources:
* Workload decision "Enough Blocks?" -- Fig. 1; stage 1 splits one
  system over several processors, stage 2 gives each system one processor
  (P:L474-493).
* Default (machine-oblivious) parameters, §IV-B: on-chip entry at 256
  elements ("the weakest architecture only able to fit 256
  elements ... we select this as our switch point"), stage 1 stops at sixteen
  independent systems.  The default Thomas switch is unstated
  ("large enough that each warp has systems to solve"): reading
  R10 takes 32.
* Machine-query ("static") parameters, §IV-C: enter the on-chip kernel as soon
  as the subsystem fits in the shared memory of ONE processor (
  Table II P:L729-730 "shared memory per processor ... limits the maximum size
  our PCR-Thomas kernel can solve"), switch to Thomas at 64 independent
  subsystems per block (2 x warp size), stage 1->2 threshold from
  the processor count only: theta = #SMs.
* Levels per HBM pass: k_p <= 9 (fp32) / 8 (fp64), passes as equal as
  possible, larger first (halo overhead <= 12.5 % of an
  n_onchip_max tile).  Segments per system: max(1, ceil(theta / M))
  (the paper's stage 1 while fewer than theta systems exist).
"""
from __future__ import annotations

from dataclasses import dataclass, field

F32, F64 = 0, 1
DEFAULT, STATIC, TUNED = 0, 1, 2
MAX_PASSES = 8

# Paper constants (cited above)
DEFAULT_NSUB_TARGET = 256
DEFAULT_THETA = 16
STATIC_THOMAS_PER_WARP = 2     # 64 = 2 x warp size
DEFAULT_THOMAS = 32            # reading R10 (P:L602-607 gives no number)
KP_MAX = {F32: 9, F64: 8}
SMEM_RESERVE = 1024            # shared memory the runtime reserves per block (device fact)


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


def n_onchip_max(props: Props, dtype: int) -> int:
    """"Switch as soon as it fits": the largest power of two n
    whose four arrays (a, b, c, d) fit in one processor's shared memory,
    4 n sizeof(T) <= smem_optin - reserve (SURVEY §8 preamble)."""
    budget = props.smem_optin_bytes - SMEM_RESERVE
    n = 1
    while 4 * (2 * n) * dsize(dtype) <= budget:
        n *= 2
    return n


@dataclass
class Plan:
    dtype: int
    mode: int
    n: int
    m: int
    n_sub_target: int = 0      # stage 2->3 switch (a subsystem size, reading R8)
    n_onchip_max: int = 0
    thomas_switch: int = 0     # stage 3->4 switch T (Thomas chains per block)
    theta: int = 0             # stage 1->2 threshold (independent systems)
    kp_max: int = 0
    k: int = 0
    n_sub: int = 0
    num_subsystems: int = 0
    passes: int = 0
    k_pass: list = field(default_factory=lambda: [0] * MAX_PASSES)
    segments: int = 0          # split segments per system (stage 1 while m < theta)


def make_plan(props: Props, dtype: int, n: int, m: int, mode: int = STATIC, kp_max: int = 0) -> Plan:
    """The method's integer plan.  ``kp_max`` overrides §8(a)'s per-pass level
    limit (a device whose shared memory cannot hold the halo of a 9-level
    pass runs shallower passes; the C++ planner reports its value)."""
    if n < 1 or m < 1:
        raise ValueError("n, m >= 1")
    if mode not in (DEFAULT, STATIC):
        raise ValueError("mode")
    p = Plan(dtype=dtype, mode=mode, n=n, m=m)
    p.n_onchip_max = n_onchip_max(props, dtype)
    if mode == DEFAULT:
        p.n_sub_target, p.thomas_switch, p.theta = DEFAULT_NSUB_TARGET, DEFAULT_THOMAS, DEFAULT_THETA
    else:
        p.n_sub_target = p.n_onchip_max
        p.thomas_switch = STATIC_THOMAS_PER_WARP * props.warp_size
        p.theta = props.sm_count
    p.kp_max = kp_max or KP_MAX[dtype]

    # Stage 2->3: split until each subsystem fits: k levels, 2^k subsystems (Fig. 3a).
    k = 0
    while cdiv(n, 1 << k) > p.n_sub_target:
        k += 1
    p.k = k
    p.n_sub = cdiv(n, 1 << k)
    p.num_subsystems = m * min(1 << k, n)
    P = cdiv(k, p.kp_max) if k > 0 else 0
    if P > MAX_PASSES:
        raise ValueError("too many passes")
    p.passes = P
    if P:
        base, extra = divmod(k, P)
        for i in range(P):
            p.k_pass[i] = base + (1 if i < extra else 0)
        # Fig. 1: several processors per system (stage 1) until theta systems exist
        p.segments = max(1, cdiv(p.theta, m))
    return p
