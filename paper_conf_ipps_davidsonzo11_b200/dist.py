"""Multi-GPU drivers over torch.distributed (NCCL on B200; gloo on CPU for tests).

Two decompositions:

* **Batch sharding** -- the m systems are independent (PAPER.md P:L291-292,
  P:L503-505): each rank solves a contiguous block of systems with the same
  integer plan; no data-path collective (``shard_range``, ``broadcast_plan``).

* **One huge system** split by contiguous row blocks (``solve_huge``).  Rank g
  owns rows [g*B, (g+1)*B).  After k_d PCR levels every residue class mod
  2^k_d is an independent tridiagonal system (Fig. 3a), but each
  class still spans every rank's rows, so a halo exchange alone cannot
  decouple the ranks (SURVEY.md §0 point 2).  The steps:

  1. halo exchange: H = 2^k_d boundary rows of a, b, c, d with rank g-1 and
     g+1 (point-to-point; ranks 0 and G-1 pad with identity rows);
  2. local split: k_d fused PCR levels over the extended block of B + 2H rows
     (``tds_split_batched`` on a split-only plan); rows [H, H+B) are exact;
  3. all-to-all: residue classes [h*q, (h+1)*q) (q = 2^k_d / G) go to rank h,
     each rank contributing its B / 2^k_d rows of every class;
  4. local solve of the q owned classes (normalised, b' = 1), each a system of
     n / 2^k_d rows (``tds_solve_batched``: more split passes + on-chip);
  5. all-to-all of x back and placement into the local rows.

The local compute is injectable (``split_fn``, ``solve_fn``) so the index
arithmetic and the collectives can be exercised on CPU with gloo against the
oracle; the defaults run libtds on the rank's GPU.
"""
from __future__ import annotations

import math
from typing import Callable, Optional, Sequence, Tuple

import torch
import torch.distributed as dist

from . import api


# ------------------------------------------------------------------ batch sharding

def shard_range(m: int, world: int, rank: int) -> Tuple[int, int]:
    """Contiguous block of systems [s0, s1) owned by `rank` (ceil(m/world) each)."""
    per = -(-m // world)
    s0 = min(m, rank * per)
    return s0, min(m, s0 + per)


def broadcast_plan(plan: api.Plan, src: int = 0, group=None, device=None) -> None:
    """Make every rank run the integer plan chosen (e.g. tuned) on `src`."""
    vals = torch.tensor(plan.params_list(), dtype=torch.int64,
                        device=device if device is not None else "cpu")
    dist.broadcast(vals, src, group=group)
    if dist.get_rank(group) != src:
        plan.set_params_list(vals.tolist())


def solve_sharded(a, b, c, d, mode: str = "static", plan: Optional[api.Plan] = None, out=None):
    """Solve this rank's block of systems ((m_local, n) CUDA tensors).  No
    collective: the systems are independent."""
    m, n = d.shape
    if plan is None:
        plan = api.Plan(n, m, str(d.dtype).replace("torch.", ""), device=d.device.index or 0, mode=mode)
    return api.solve_batched(plan, a, b, c, d, out=out)


# ------------------------------------------------------------------ one huge system

def _gpu_split(a, b, c, d, kd: int):
    """k_d PCR levels over (1, E) arrays on the GPU; canonical order, b' = 1."""
    E = d.shape[-1]
    plan = api.Plan(E, 1, str(d.dtype).replace("torch.", ""), device=d.device.index or 0, mode="static")
    plan.set_params(k_pass=_schedule(kd), split_only=1, cluster=1, tl_levels=0)
    return api.split_batched(plan, a.reshape(1, E), b.reshape(1, E), c.reshape(1, E), d.reshape(1, E))


def _gpu_solve(a, b, c, d):
    m, n = d.shape
    plan = api.Plan(n, m, str(d.dtype).replace("torch.", ""), device=d.device.index or 0, mode="static")
    return api.solve_batched(plan, a.contiguous(), b.contiguous(), c.contiguous(), d.contiguous())


def _schedule(k: int, kpmax: int = 4) -> list:
    P = -(-k // kpmax)
    return [k // P + (1 if i < k % P else 0) for i in range(P)]


def huge_kd(world: int, kd: Optional[int] = None) -> int:
    """Levels split before the exchange: at least log2(world) so every rank owns a class."""
    base = max(1, int(math.ceil(math.log2(world)))) if world > 1 else 1
    return max(base, kd or 0)


def solve_huge(a_loc, b_loc, c_loc, d_loc, n: int, group=None, kd: Optional[int] = None,
               split_fn: Callable = _gpu_split, solve_fn: Callable = _gpu_solve):
    """Solve one system of n rows whose row block [g*B, (g+1)*B) lives on rank g.

    a_loc .. d_loc: 1-D tensors of B = n / G rows (the rank's block; a_0 and
    c_{n-1} of the global system are ignored).  Returns x for the local rows.
    Requirements: G a power of two, B a multiple of 2^k_d.
    """
    G = dist.get_world_size(group) if dist.is_initialized() else 1
    g = dist.get_rank(group) if dist.is_initialized() else 0
    kd = huge_kd(G, kd)
    NR = 1 << kd
    B = d_loc.shape[-1]
    if G & (G - 1) or B * G != n or B % NR:
        raise ValueError(f"solve_huge: need G a power of two, n = G*B, B % 2^kd == 0 (G={G}, n={n}, kd={kd})")
    H = NR                      # halo rows per side (>= 2^kd - 1, aligned to the residue period)
    dev, dt = d_loc.device, d_loc.dtype
    loc = torch.stack([a_loc, b_loc, c_loc, d_loc])  # (4, B)
    if g == 0:
        loc[0, 0] = 0
    if g == G - 1:
        loc[2, B - 1] = 0

    # 1. halo exchange with g-1 / g+1
    ident = torch.zeros(4, H, dtype=dt, device=dev)
    ident[1] = 1
    left, right = ident.clone(), ident.clone()
    if G > 1:
        ops = []
        if g > 0:
            ops.append(dist.P2POp(dist.isend, loc[:, :H].contiguous(), g - 1, group))
            ops.append(dist.P2POp(dist.irecv, left, g - 1, group))
        if g < G - 1:
            ops.append(dist.P2POp(dist.isend, loc[:, B - H:].contiguous(), g + 1, group))
            ops.append(dist.P2POp(dist.irecv, right, g + 1, group))
        for r in dist.batch_isend_irecv(ops):
            r.wait()
    ext = torch.cat([left, loc, right], dim=1)  # (4, E), E = B + 2H; ext row e = global row g*B - H + e

    # 2. local split (k_d levels); canonical order: residue r, position j (ext row r + NR*j)
    sa, sc, sd = split_fn(ext[0], ext[1], ext[2], ext[3], kd)
    E = B + 2 * H
    per = E // NR                                # rows per residue in the extended block
    Bj = B // NR                                 # valid rows per residue (positions 1 .. Bj)
    split = torch.stack([sa.reshape(NR, per), sc.reshape(NR, per), sd.reshape(NR, per)])  # (3, NR, per)
    valid = split[:, :, H // NR: H // NR + Bj]   # (3, NR, Bj)

    # 3. all-to-all: residues [h*q, (h+1)*q) -> rank h
    q = NR // G
    send = valid.reshape(3, G, q, Bj).permute(1, 0, 2, 3).contiguous()  # (G, 3, q, Bj)
    recv = torch.empty_like(send)
    if G > 1:
        dist.all_to_all_single(recv, send, group=group)
    else:
        recv.copy_(send)
    # recv[src]: rows j-block src of my q residues -> (3, q, G*Bj) systems
    sys = recv.permute(1, 2, 0, 3).reshape(3, q, G * Bj)

    # 4. local solve of the owned residue systems (normalised: b' = 1)
    ones = torch.ones_like(sys[0])
    xs = solve_fn(sys[0].contiguous(), ones, sys[1].contiguous(), sys[2].contiguous())  # (q, n/NR)

    # 5. x back: rank h returns j-block g of its residues to rank g
    xsend = xs.reshape(q, G, Bj).permute(1, 0, 2).contiguous()  # (G, q, Bj)
    xrecv = torch.empty_like(xsend)
    if G > 1:
        dist.all_to_all_single(xrecv, xsend, group=group)
    else:
        xrecv.copy_(xsend)
    # xrecv[h][rl][jj] = x of global row (h*q + rl) + NR*(g*Bj + jj) = local row (h*q+rl) + NR*jj
    x_loc = xrecv.reshape(NR, Bj).t().contiguous().reshape(B)
    return x_loc


def huge_bytes(n: int, world: int, s: int = 4, kd: Optional[int] = None) -> dict:
    """Bytes each rank moves over the interconnect in solve_huge."""
    kd = huge_kd(world, kd)
    B = n // world
    return {"halo": 2 * 4 * (1 << kd) * s if world > 1 else 0,
            "all_to_all_split": 3 * B * s * (world - 1) // world,
            "all_to_all_x": B * s * (world - 1) // world}
