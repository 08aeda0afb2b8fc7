"""Multi-GPU drivers over torch.distributed (NCCL on B200; gloo on CPU for tests).

Two decompositions:

* **Batch sharding** -- the m systems are independent (PAPER.md P:L291-292,
  P:L503-505): each rank solves a contiguous block of systems with the same
  integer plan; no data-path collective (``shard_range``, ``broadcast_plan``).

* **One huge system** split by contiguous row blocks (``HugeRank`` /
  ``solve_huge``) -- the paper's Stage 1, several processors cooperating on one
  system, lifted to several GPUs.  Rank g owns rows [g B, (g+1) B)
  inside a halo-padded block ``ext`` of E = B + 2H rows (global rows
  g B - H .. g B + B + H; identity rows (0, 1, 0, 0) outside [0, n)).  After
  k_d PCR levels every residue class mod 2^k_d is an independent system
  (Fig. 3a), but each class still spans every rank's rows, so a
  halo exchange alone cannot decouple the ranks (SURVEY.md §0 point 2):

  1. halo exchange: H rows of a, b, c, d with ranks g-1 and g+1, received
     straight into ext's padding (point-to-point, no copy);
  2. local split: k_d fused PCR levels over ext (``tds_split_slots``): the
     split system stays in the workspace, residue r of the block in slot r,
     rows [H, H + B) of ext exact (H >= 2^k_d - 1);
  3. all-to-all: residue classes [h q, (h+1) q) (q = 2^k_d / G) go to rank h.
     Every (array, residue) run of the block is ONE contiguous slot segment, so
     the sends read the split's slots in place and the receives land in place
     in the destination's residue systems -- no pack / unpack copies (only the
     rank's own 1/G share is copied locally);
  4. local solve of the q owned residue systems (normalised, b' = 1:
     ``tds_solve_normalized``, no b array), in ``chunks`` groups of residues:
     group c is solved while group c+1 is still arriving;
  5. x return: the solve's x runs go back to their owners (again contiguous
     segments on both sides), then ONE residue->row transpose
     (``tds_unpack_residues``, the placement kernel) writes x in row order.

  With G = 1 there is nothing to exchange: the residue systems are read in
  place from the split's slots (a slot view with batch_stride = slot_rows).

The communication is a generator protocol: ``huge_steps`` yields at every
exchange, so the same code runs over torch.distributed point-to-point ops
(``P2PTransport``: NCCL on GPUs, gloo on CPU) or over the G ranks of a
single-GPU loopback world (``solve_huge_loopback``: every rank's buffers and
kernels on one device, messages as device copies) -- the full multi-rank data
path exercised with the real kernels on one GPU.  The local compute is a
backend object (``CudaBackend`` runs libtds; the gloo tests plug in the CPU
oracle).
"""
from __future__ import annotations

import math
from typing import Callable, List, Optional, Sequence, Tuple

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

def huge_kd(world: int, kd: Optional[int] = None) -> int:
    """Levels split before the exchange: at least log2(world) so every rank owns a class."""
    base = max(1, int(math.ceil(math.log2(world)))) if world > 1 else 1
    return max(base, kd or 0)


def huge_halo(kd: int, itemsize: int) -> int:
    """Halo rows per side: >= 2^k_d - 1 (exactness of k_d fused levels), a
    multiple of 2^k_d (residues of ext rows = residues of global rows) and of
    16 bytes per residue (the G = 1 slot views stay 16-byte aligned)."""
    return (1 << kd) * max(1, 16 // itemsize)


def _schedule(k: int, kpmax: int = 8) -> list:
    P = -(-k // kpmax)
    return [k // P + (1 if i < k % P else 0) for i in range(P)]


class CudaBackend:
    """libtds on this rank's GPU: split to slots, normalised solves, x unpack."""

    def __init__(self, dtype: torch.dtype, device, mode: str = "static"):
        self.dtype, self.device, self.mode = dtype, torch.device(device), mode
        self.name = str(dtype).replace("torch.", "")

    def empty(self, *shape):
        return torch.empty(*shape, dtype=self.dtype, device=self.device)

    def make_split(self, E: int, kd: int):
        plan = api.Plan(E, 1, self.name, device=self.device.index or 0, mode="static")
        plan.set_params(k_pass=_schedule(kd), split_only=1, cluster=1, tl_levels=0)
        ws = plan.workspace()
        return plan, ws, api.slot_views(plan, ws)

    def split(self, state, ext):
        plan, ws, _ = state
        api.split_slots(plan, ext[0], ext[1], ext[2], ext[3], ws)

    def split_scatter(self, state, ext, dst, q: int, first_pos: int, num_pos: int, dst_stride: int):
        """The split with the all-to-all fused into its TMA stores (tds_split_scatter)."""
        plan = state[0]
        api.split_scatter(plan, ext[0], ext[1], ext[2], ext[3], dst, q, first_pos, num_pos, dst_stride)

    def x_fusable(self, state, Bj: int) -> bool:
        """Whether the residue solve can place x straight into the owners
        (tds_solve_normalized_xscatter's shape rules)."""
        info = state[0].info
        k, E = info["k"], 128 // torch.empty((), dtype=self.dtype).element_size()
        return (k >= 5 and info["chunks"] == 1 and info["x_group"] == 0 and info["strided"] == 0 and
                info["n"] % (1 << k) == 0 and Bj % (1 << k) == 0 and (Bj >> k) % (4 * E) == 0)

    def solve_xscatter(self, state, a, c, d, dst, Bj: int):
        plan, ws = state
        api.solve_normalized_xscatter(plan, a, c, d, dst, Bj, Bj, workspace=ws)

    def make_solve(self, NL: int, m: int, stride: int):
        plan = api.Plan(NL, m, self.name, device=self.device.index or 0, mode="static", batch_stride=stride)
        if plan.info["k"] == 0:
            # normalised input needs >= 1 split level (the k = 0 kernels read b): one level, the
            # static on-chip shape for the halved subsystems
            T0 = plan.info["thomas_chains"]
            for T in [T0] + [t for t in (32, 16, 8, 4, 2, 1) if t < T0]:
                try:
                    plan.set_params(k_pass=[1], cluster=1, tl_levels=0, thomas_chains=T)
                    break
                except api.L.TdsError:
                    continue
        return plan, plan.workspace()

    def solve(self, state, a, c, d, x):
        plan, ws = state
        api.solve_normalized(plan, a, c, d, out=x, workspace=ws)

    def unpack(self, xs, out, B: int, kd: int, slot_rows: int):
        api.unpack_residues(xs, out, B, 1, kd, slot_rows)

    def make_full(self, n: int, kd: int, res_plan):
        """G = 1: the k_d-level split and the residue solves as ONE plan --
        passes [k_d] + the residue plan's, the residue plan's on-chip shape --
        so x is placed straight into row order (no x slots round trip, no
        unpack).  Same per-row arithmetic as the split + residue solves."""
        p = res_plan.info
        plan = api.Plan(n, 1, self.name, device=self.device.index or 0, mode="static")
        keys = ("cr_levels", "thomas_chains", "cluster", "tl_levels", "split_tile_rows", "split_threads", "theta")
        kw = {k: p[k] for k in keys}
        try:
            plan.set_params(k_pass=_schedule(kd) + p["k_pass"], x_group=p["x_group"], **kw)
        except api.L.TdsError:
            plan.set_params(k_pass=_schedule(kd) + p["k_pass"], x_group=0, **kw)
        return plan, plan.workspace()

    def solve_full(self, state, ext, H: int, n: int, out):
        plan, ws = state
        api.solve_batched(plan, *(ext[t, H:H + n] for t in range(4)), out=out, workspace=ws)


class HugeRank:
    """One rank's buffers, plans and message lists for ``huge_steps`` (all
    allocated once; a solve only enqueues kernels and exchanges)."""

    def __init__(self, n: int, G: int, g: int, backend, kd: Optional[int] = None, chunks: int = 1,
                 sys_alloc: Optional[Callable] = None):
        """``sys_alloc(shape)``: allocator of the residue-system buffer (3, q, NL)
        -- e.g. torch symmetric memory, so peers can write into it (peer mode,
        ``set_peers``); default: the backend's allocator."""
        itemsize = torch.empty((), dtype=backend.dtype).element_size()
        self.n, self.G, self.g, self.be = n, G, g, backend
        self.peer_dst = None                     # peer mode: tds_scatter destinations (set_peers)
        self.x_fused = False                     # peer mode: x placed straight into its owners
        self.kd = kd = huge_kd(G, kd)
        self.NR = NR = 1 << kd
        self.B = B = n // G
        if G & (G - 1) or B * G != n or B % NR or NR % G:
            raise ValueError(f"solve_huge: need G a power of two, n = G B, B % 2^kd == 0, 2^kd % G == 0 "
                             f"(G={G}, n={n}, kd={kd})")
        self.q = q = NR // G                     # residue classes (local systems) per rank
        if q % chunks:
            raise ValueError(f"chunks ({chunks}) must divide the {q} residue systems per rank")
        self.chunks = chunks
        self.H = H = huge_halo(kd, itemsize)
        self.E = E = B + 2 * H
        self.Bj = Bj = B // NR                   # rows of one residue class inside the block
        self.NL = NL = n // NR                   # rows of one residue system
        self.off = H // NR                       # first valid position of each slot
        self.ext = backend.empty(4, E)           # a, b, c, d of global rows gB - H .. gB + B + H
        self.ext.zero_()
        self.ext[1].fill_(1)                     # identity rows until the halo arrives (stay at the ends)
        self.split_state = backend.make_split(E, kd)
        self.slots = self.split_state[2]         # (a', c', d') as (NR, stride) views
        self.stride = self.slots[0].shape[1]
        qc = q // chunks
        if G == 1:
            # the residue systems are read in place from the slots (batch_stride = slot stride)
            flat = [v.reshape(-1) for v in self.slots]
            self.sys = None
            span = (qc - 1) * self.stride + NL
            self.chunk_in = [tuple(f[self.off + c * qc * self.stride:][:span] for f in flat) for c in range(chunks)]
            self.solve_states = [backend.make_solve(NL, qc, self.stride) for _ in range(chunks)]
        else:
            # one buffer: the residue systems (3, q, NL) and the returned x (NR, Bj) -- in peer
            # mode both are written by the peers' kernels (symmetric memory on a multi-GPU node)
            nsys = 3 * q * NL
            self.sys_buf = sys_alloc((nsys + NR * Bj,)) if sys_alloc else backend.empty(nsys + NR * Bj)
            self.sys = [self.sys_buf[t * q * NL:(t + 1) * q * NL].view(q, NL) for t in range(3)]
            self.chunk_in = [tuple(v[c * qc:(c + 1) * qc] for v in self.sys) for c in range(chunks)]
            self.solve_states = [backend.make_solve(NL, qc, NL) for _ in range(chunks)]
        # x of the local residue systems (G = 1: with the slots' stride, unpacked in place)
        self.xs = backend.empty(q, self.stride if G == 1 else NL)
        self.chunk_x = [self.xs[c * qc:(c + 1) * qc] for c in range(chunks)]
        self.xrecv = self.xs if G == 1 else self.sys_buf[3 * q * NL:].view(NR, Bj)
        # G = 1 with a backend that can fuse: split + residue solves as one plan
        self.full = backend.make_full(n, kd, self.solve_states[0][0]) if G == 1 and hasattr(backend, "make_full") \
            else None

    def set_peers(self, sys_ptrs: Sequence[int]) -> None:
        """Peer mode: ``sys_ptrs[h]`` = device address (peer-mapped for h != g)
        of rank h's residue-system buffer (3, q, NL).  The split then writes
        every residue class straight into its owner (tds_split_scatter): the
        all-to-all of the split data is fused into the split's TMA stores."""
        s = self.ext.element_size()
        q, NL, Bj, g = self.q, self.NL, self.Bj, self.g
        self.peer_dst = [[int(sys_ptrs[h]) + (t * q * NL + g * Bj) * s for h in range(self.G)] for t in range(3)]
        # x: chunk c's systems [c qc, (c+1) qc) -> rows g q + c qc ... of every owner's returned-x block
        qc = q // self.chunks
        self.peer_xdst = [[int(sys_ptrs[h]) + (3 * q * NL + (g * q + c * qc) * Bj) * s for h in range(self.G)]
                          for c in range(self.chunks)]
        self.x_fused = all(self.be.x_fusable(st_, Bj) for st_ in self.solve_states) if hasattr(self.be, "x_fusable") \
            else False

    @property
    def local(self):
        """(a, b, c, d) views of the rank's own rows (fill them before solving)."""
        return tuple(self.ext[t, self.H:self.H + self.B] for t in range(4))

    # -------- message lists: (peer, tensor) in the order both sides post them
    def halo_messages(self):
        H, B, E, g = self.H, self.B, self.E, self.g
        sends, recvs = [], []
        if g > 0:
            sends += [(g - 1, self.ext[t, H:2 * H]) for t in range(4)]
            recvs += [(g - 1, self.ext[t, 0:H]) for t in range(4)]
        if g < self.G - 1:
            sends += [(g + 1, self.ext[t, B:B + H]) for t in range(4)]
            recvs += [(g + 1, self.ext[t, B + H:E]) for t in range(4)]
        return sends, recvs

    def _chunk(self, c):
        qc = self.q // self.chunks
        return range(c * qc, (c + 1) * qc)

    def a2a_messages(self, c):
        sends, recvs, local = [], [], []
        o, Bj, q, g = self.off, self.Bj, self.q, self.g
        for h in range(self.G):
            for t in range(3):
                for rl in self._chunk(c):
                    seg_out = self.slots[t][h * q + rl, o:o + Bj]        # my rows of residue h q + rl
                    seg_in = self.sys[t][rl, h * Bj:(h + 1) * Bj]        # rank h's rows of my residue rl
                    if h == g:
                        local.append((seg_out, seg_in))
                    else:
                        sends.append((h, seg_out))
                        recvs.append((h, seg_in))
        return sends, recvs, local

    def xret_messages(self, c):
        sends, recvs, local = [], [], []
        Bj, q, g = self.Bj, self.q, self.g
        for h in range(self.G):
            for rl in self._chunk(c):
                seg_out = self.xs[rl, h * Bj:(h + 1) * Bj]               # x of my residue rl, rank h's rows
                seg_in = self.xrecv[h * q + rl]                           # x of residue h q + rl, my rows
                if h == g:
                    local.append((seg_out, seg_in))
                else:
                    sends.append((h, seg_out))
                    recvs.append((h, seg_in))
        return sends, recvs, local

    # -------- residue-solve plan (all chunks share one shape)
    def residue_params(self) -> list:
        return self.solve_states[0][0].params_list()

    def set_residue_params(self, vals) -> None:
        """Apply one integer plan to every chunk's residue solve (e.g. tuned on
        rank 0 and broadcast); a plan with k = 0 (normalised input needs a
        split level) is refused by tds_solve_normalized, so it is not applied."""
        new = []
        for plan, _ in self.solve_states:
            old = plan.params_list()
            plan.set_params_list(vals)
            if plan.info["k"] == 0:
                plan.set_params_list(old)
            new.append((plan, plan.workspace()))
        self.solve_states = new
        if self.full is not None:
            self.full = self.be.make_full(self.n, self.kd, self.solve_states[0][0])
        if self.peer_dst is not None and hasattr(self.be, "x_fusable"):
            self.x_fused = all(self.be.x_fusable(st_, self.Bj) for st_ in self.solve_states)

    def tune_residues(self, cache_path=None) -> list:
        """tds_tune on the residue-solve shape (this rank's device); applied to
        every chunk.  Returns the integer plan (to broadcast)."""
        plan = self.solve_states[0][0]
        before = plan.params_list()
        plan.tune(cache_path=cache_path)
        vals = plan.params_list()
        plan.set_params_list(before)
        self.set_residue_params(vals)
        return self.residue_params()

    # -------- compute
    def split(self):
        self.be.split(self.split_state, self.ext)

    def solve(self, c):
        a, cc, d = self.chunk_in[c]
        self.be.solve(self.solve_states[c], a, cc, d, self.chunk_x[c])

    def unpack(self, out):
        self.be.unpack(self.xrecv, out, self.B, self.kd, self.xrecv.shape[1])


def huge_steps(R: HugeRank, out, mark=None):
    """One solve of rank R's part; a generator that yields ("post", sends,
    recvs) and ("wait", handle) at every exchange (the driver performs them).
    ``mark(phase)`` (optional) is called at the phase boundaries "halo",
    "split", "exchange_solve", "unpack", "end" (per-phase event timing)."""
    mark = mark or (lambda phase: None)
    mark("halo")
    if R.G > 1:
        h = yield ("post",) + R.halo_messages()
        yield ("wait", h)
    mark("split")
    if R.peer_dst is not None and R.G > 1:  # peer mode: split + all-to-all in one kernel, then a barrier
        R.be.split_scatter(R.split_state, R.ext, R.peer_dst, R.q, R.off, R.Bj, R.NL)
        mark("exchange_solve")
        yield ("barrier",)                  # every rank's split has written into every owner
        if R.x_fused:  # the placement writes x straight into its owners' blocks, then a barrier
            for c in range(R.chunks):
                a, cc, d = R.chunk_in[c]
                R.be.solve_xscatter(R.solve_states[c], a, cc, d, R.peer_xdst[c], R.Bj)
            yield ("barrier",)
            mark("unpack")
            R.unpack(out)
            mark("end")
            return out
        for c in range(R.chunks):
            R.solve(c)
        xret = []
        for c in range(R.chunks):
            sends, recvs, local = R.xret_messages(c)
            xret.append((yield ("post", sends, recvs)))
            for src, dst in local:
                dst.copy_(src)
        for c in range(R.chunks):
            yield ("wait", xret[c])
        mark("unpack")
        R.unpack(out)
        mark("end")
        return out
    if R.full is not None:  # G = 1, fused: one plan, x straight into row order
        R.be.solve_full(R.full, R.ext, R.H, R.n, out)
        mark("exchange_solve")
        mark("unpack")
        mark("end")
        return out
    R.split()
    mark("exchange_solve")
    if R.G > 1:
        a2a = []
        for c in range(R.chunks):
            sends, recvs, local = R.a2a_messages(c)
            a2a.append((yield ("post", sends, recvs)))
            for src, dst in local:
                dst.copy_(src)
        xret = []
        for c in range(R.chunks):
            yield ("wait", a2a[c])
            R.solve(c)
            sends, recvs, local = R.xret_messages(c)
            xret.append((yield ("post", sends, recvs)))
            for src, dst in local:
                dst.copy_(src)
        for c in range(R.chunks):
            yield ("wait", xret[c])
    else:
        for c in range(R.chunks):
            R.solve(c)
    mark("unpack")
    R.unpack(out)
    mark("end")
    return out


class P2PTransport:
    """torch.distributed point-to-point (batch_isend_irecv): NCCL on GPUs (the
    ops run on NCCL's stream, ordered after the current stream's kernels and
    waited on by it), gloo on CPU."""

    def __init__(self, group=None, symm=None):
        """``symm``: a torch symmetric-memory handle of the peer-mode residue
        buffers -- its device-side barrier orders the peers' fused split
        stores before the residue solves (else a process-group barrier)."""
        self.group, self.symm = group, symm

    def barrier(self):
        if self.symm is not None:
            self.symm.barrier()
        else:
            dist.barrier(group=self.group)

    def post(self, sends, recvs):
        ops = [dist.P2POp(dist.isend, t, peer, self.group) for peer, t in sends]
        ops += [dist.P2POp(dist.irecv, t, peer, self.group) for peer, t in recvs]
        return dist.batch_isend_irecv(ops) if ops else []

    @staticmethod
    def wait(works):
        for w in works:
            w.wait()


def run_steps(gen, transport: P2PTransport):
    """Drive one rank's ``huge_steps`` generator over a real transport."""
    try:
        msg = next(gen)
        while True:
            if msg[0] == "post":
                msg = gen.send(transport.post(msg[1], msg[2]))
            elif msg[0] == "barrier":
                transport.barrier()
                msg = gen.send(None)
            else:
                transport.wait(msg[1])
                msg = gen.send(None)
    except StopIteration as e:
        return e.value


def solve_huge_loopback(ranks: Sequence[HugeRank], outs: Sequence):
    """Run G ranks' ``huge_steps`` in ONE process (one device): a message from
    rank g to rank h is a copy from g's send tensor to h's receive tensor,
    matched in posting order per (g, h) pair exactly as NCCL matches them."""
    G = len(ranks)
    gens = [huge_steps(R, o) for R, o in zip(ranks, outs)]
    pending = {}                                   # (src, dst) -> [sends], [recvs]
    state, done = [None] * G, [False] * G
    for g, gen in enumerate(gens):
        try:
            state[g] = next(gen)
        except StopIteration:                      # G = 1: nothing to exchange
            done[g] = True
    while not all(done):
        progressed = False
        for g in range(G):
            while not done[g] and state[g][0] == "post":
                _, sends, recvs = state[g]
                for peer, t in sends:
                    pending.setdefault((g, peer), ([], []))[0].append(t)
                for peer, t in recvs:
                    pending.setdefault((peer, g), ([], []))[1].append(t)
                try:
                    state[g] = gens[g].send(None)
                except StopIteration:
                    done[g] = True
                progressed = True
        # every rank is waiting (or done): deliver every matched message
        for key, (sends, recvs) in pending.items():
            k = min(len(sends), len(recvs))
            for src, dst in zip(sends[:k], recvs[:k]):
                assert src.numel() == dst.numel(), key
                dst.copy_(src)
            del sends[:k], recvs[:k]
        for g in range(G):
            if not done[g] and state[g][0] == "wait":
                try:
                    state[g] = gens[g].send(None)
                except StopIteration:
                    done[g] = True
                progressed = True
        # a barrier releases only when every live rank has reached it
        live = [g for g in range(G) if not done[g]]
        if live and all(state[g][0] == "barrier" for g in live):
            for g in live:
                try:
                    state[g] = gens[g].send(None)
                except StopIteration:
                    done[g] = True
            progressed = True
        if not progressed:
            raise RuntimeError("loopback deadlock")
    return outs


def solve_huge(a_loc, b_loc, c_loc, d_loc, n: int, group=None, kd: Optional[int] = None, backend=None,
               chunks: int = 1, rank_state: Optional[HugeRank] = None):
    """Solve one system of n rows whose row block [g B, (g+1) B) lives on rank
    g (1-D tensors of B rows; a_0 and c_{n-1} of the global system are
    ignored).  Returns x for the local rows.  ``rank_state`` reuses the
    buffers and plans of an earlier call (allocate once with ``HugeRank``)."""
    G = dist.get_world_size(group) if dist.is_initialized() else 1
    g = dist.get_rank(group) if dist.is_initialized() else 0
    if backend is None:
        backend = CudaBackend(d_loc.dtype, d_loc.device)
    R = rank_state or HugeRank(n, G, g, backend, kd=kd, chunks=chunks)
    for dst, src in zip(R.local, (a_loc, b_loc, c_loc, d_loc)):
        dst.copy_(src)
    out = backend.empty(R.B)
    return run_steps(huge_steps(R, out), P2PTransport(group))


def huge_bytes(n: int, world: int, s: int = 4, kd: Optional[int] = None) -> dict:
    """Bytes each rank moves over the interconnect in solve_huge (NVLink)."""
    kd = huge_kd(world, kd)
    B = n // world
    H = huge_halo(kd, s)
    return {"halo": 2 * 4 * H * s if world > 1 else 0,
            "all_to_all_split": 3 * B * s * (world - 1) // world,
            "all_to_all_x": B * s * (world - 1) // world}
