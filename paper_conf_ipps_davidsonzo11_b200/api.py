"""Python face of libtds: the same names as the C ABI (include/tds.h).

Argument marshalling only -- every step of the solve runs in libtds's sm_100a
kernels.  PyTorch supplies device memory (tensors) and streams.
"""
from __future__ import annotations

import ctypes
from typing import Optional

import numpy as np

from . import _lib as L

_DTYPES = {"float32": L.TDS_F32, "float64": L.TDS_F64}
MODES = {"default": L.TDS_PARAMS_DEFAULT, "static": L.TDS_PARAMS_STATIC, "tuned": L.TDS_PARAMS_TUNED}


def _dtype_code(dtype) -> int:
    name = str(dtype).replace("torch.", "")
    if name not in _DTYPES:
        raise TypeError(f"unsupported dtype {dtype}: float32 or float64")
    return _DTYPES[name]


def _stream_ptr(stream, device: Optional[int] = None) -> Optional[int]:
    import torch
    if stream is None:
        if device is not None:  # the raw current-stream handle, without building a Stream object
            return torch._C._cuda_getCurrentRawStream(device)
        stream = torch.cuda.current_stream()
    return stream.cuda_stream


def device_props(device: int = 0) -> dict:
    lib = L.load()
    p = L.DeviceProps()
    L.check(lib.tds_device_props_query(int(device), ctypes.byref(p)))
    return {f: getattr(p, f) for f, _ in L.DeviceProps._fields_}


def params_to_dict(p: L.Params) -> dict:
    return {"k": p.k, "passes": p.passes, "k_pass": list(p.k_pass)[: max(p.passes, 0)],
            "cr_levels": p.cr_levels, "thomas_chains": p.thomas_chains, "cluster": p.cluster,
            "tl_levels": p.tl_levels, "chunk_systems": p.chunk_systems,
            "split_tile_rows": p.split_tile_rows, "split_threads": p.split_threads, "theta": p.theta,
            "x_group": p.x_group, "strided": p.strided}


class Plan:
    """tds_plan / tds_plan_from_props wrapper (host object; owns no device memory)."""

    def __init__(self, n: int, m: int, dtype="float32", device: int = 0, mode: str = "static",
                 batch_stride: int = 0, props: Optional[dict] = None):
        self._lib = L.load()
        self._h = ctypes.c_void_p()
        code = _dtype_code(dtype)
        if props is not None:
            dp = L.DeviceProps(**props)
            L.check(self._lib.tds_plan_from_props(ctypes.byref(self._h), ctypes.byref(dp), code, int(n),
                                                  int(m), int(batch_stride), MODES[mode]))
        else:
            L.check(self._lib.tds_plan(ctypes.byref(self._h), int(device), code, int(n), int(m),
                                       int(batch_stride), MODES[mode]))
        self.dtype = "float32" if code == L.TDS_F32 else "float64"

    def __del__(self):
        h = getattr(self, "_h", None)
        if h is not None and h.value:
            self._lib.tds_plan_destroy(h)
            self._h = None

    @property
    def handle(self):
        return self._h

    def info_struct(self) -> L.PlanInfo:
        info = L.PlanInfo()
        L.check(self._lib.tds_plan_info_get(self._h, ctypes.byref(info)))
        return info

    def _solve_info(self):
        """(info, required elements, torch dtype, device), cached per plan state
        (set_params / set_params_list / tune drop it)."""
        c = getattr(self, "_cache", None)
        if c is None:
            import torch
            info = self.info_struct()
            c = (info, (info.m - 1) * info.batch_stride + info.n,
                 torch.float32 if info.dtype == L.TDS_F32 else torch.float64, int(info.device))
            self._cache = c
        return c

    @property
    def info(self) -> dict:
        s = self.info_struct()
        out = {f: getattr(s, f) for f, _ in L.PlanInfo._fields_ if f not in ("params", "pad_")}
        out.update(params_to_dict(s.params))
        return out

    @property
    def params(self) -> L.Params:
        return self.info_struct().params

    @property
    def workspace_bytes(self) -> int:
        return int(self.info_struct().workspace_bytes)

    def set_params(self, **kw) -> None:
        """tds_plan_set_params: replace tunables (k, k_pass, cr_levels, thomas_chains, ...)."""
        p = self.params
        for key, val in kw.items():
            if key == "k_pass":
                vals = list(val) + [0] * (L.TDS_MAX_PASSES - len(val))
                for i in range(L.TDS_MAX_PASSES):
                    p.k_pass[i] = vals[i]
                p.passes = len(val)
                p.k = sum(val)
            else:
                setattr(p, key, int(val))
        self._cache = None
        L.check(self._lib.tds_plan_set_params(self._h, ctypes.byref(p)))

    def params_list(self) -> list:
        """All tunable integers (tds_params field order) -- e.g. to broadcast a
        tuned plan from rank 0 so every rank runs identical kernels."""
        p = self.params
        out = []
        for f, _ in L.Params._fields_:
            v = getattr(p, f)
            out.extend(list(v) if f == "k_pass" else [v])
        return out

    def set_params_list(self, vals) -> None:
        p = L.Params()
        it = iter(int(v) for v in vals)
        for f, _ in L.Params._fields_:
            if f == "k_pass":
                for i in range(L.TDS_MAX_PASSES):
                    p.k_pass[i] = next(it)
            else:
                setattr(p, f, next(it))
        self._cache = None
        L.check(self._lib.tds_plan_set_params(self._h, ctypes.byref(p)))

    def permutation(self) -> np.ndarray:
        n = self.info_struct().n
        out = np.empty(n, dtype=np.int64)
        L.check(self._lib.tds_plan_permutation(self._h, out.ctypes.data, int(n)))
        return out

    def tune(self, stream=None, cache_path: Optional[str] = None) -> int:
        """tds_tune; returns the number of timed trials (0 on a cache hit)."""
        cp = cache_path.encode() if cache_path else None
        self._cache = None
        L.check(self._lib.tds_tune(self._h, _stream_ptr(stream), cp))
        t = ctypes.c_int32()
        L.check(self._lib.tds_plan_tune_trials(self._h, ctypes.byref(t)))
        return int(t.value)

    def tune_search(self, cost, cache_path: Optional[str] = None) -> int:
        """tds_tune_search (TEST-ONLY): the tuner's search with ``cost(params
        dict) -> float`` in place of timed device solves.  Returns the number
        of cost calls (0 on a cache hit)."""
        def cb(p, _user):
            return float(cost(params_to_dict(p.contents)))
        fn = L.COST_FN(cb)
        cp = cache_path.encode() if cache_path else None
        self._cache = None
        L.check(self._lib.tds_tune_search(self._h, fn, None, cp))
        t = ctypes.c_int32()
        L.check(self._lib.tds_plan_tune_trials(self._h, ctypes.byref(t)))
        return int(t.value)

    @property
    def interleaved_workspace_bytes(self) -> int:
        """tds_interleaved_workspace_bytes (dense plans only)."""
        v = ctypes.c_size_t()
        L.check(self._lib.tds_interleaved_workspace_bytes(self._h, ctypes.byref(v)))
        return int(v.value)

    def slots_layout(self) -> dict:
        """tds_plan_slots_layout: where tds_split_slots leaves the split system
        in the workspace (element offsets of a', c', d', slot_rows, num_slots)."""
        lay = L.SlotsLayout()
        L.check(self._lib.tds_plan_slots_layout(self._h, ctypes.byref(lay)))
        return {f: int(getattr(lay, f)) for f, _ in L.SlotsLayout._fields_}

    def workspace(self):
        import torch
        nbytes = self.workspace_bytes
        if nbytes == 0:
            return None
        return torch.empty(nbytes, dtype=torch.uint8, device=f"cuda:{self.info_struct().device}")


def _ptr(t) -> int:
    return t.data_ptr()


def _check_tensor(t, plan_info, name):
    import torch
    want = torch.float32 if plan_info.dtype == L.TDS_F32 else torch.float64
    need = (plan_info.m - 1) * plan_info.batch_stride + plan_info.n
    _check_fast(t, need, want, name, int(plan_info.device))


def _check_fast(t, need, want, name, dev=None):
    """Argument checks of the Python face (the C ABI re-checks pointers / sizes);
    ``dev``: the plan's device -- a tensor on another GPU is refused here (the
    kernels would fault on it)."""
    if getattr(t, "is_cuda", False) is not True:
        raise TypeError(f"{name} must be a CUDA tensor")
    if dev is not None and t.device.index != dev:
        raise ValueError(f"{name} is on cuda:{t.device.index}, the plan on cuda:{dev}")
    if t.dtype != want:
        raise TypeError(f"{name} has dtype {t.dtype}, plan expects {want}")
    if t.numel() < need or not t.is_contiguous():
        raise ValueError(f"{name} must be contiguous with >= {need} elements")


def solve_batched(plan: Plan, a, b, c, d, out=None, workspace=None, stream=None):
    """x = A^{-1} d for every system (tds_solve_batched).  a, b, c, d: CUDA
    tensors laid out as the plan says (m x batch_stride).  Returns x."""
    import torch
    info, need, want, dev = plan._solve_info()
    _check_fast(a, need, want, "a", dev)
    _check_fast(b, need, want, "b", dev)
    _check_fast(c, need, want, "c", dev)
    _check_fast(d, need, want, "d", dev)
    if out is None:
        out = torch.empty_like(d)
    else:
        _check_fast(out, need, want, "out", dev)
    if workspace is None and info.workspace_bytes > 0:
        workspace = plan.workspace()
    wptr = workspace.data_ptr() if workspace is not None else None
    wbytes = workspace.numel() * workspace.element_size() if workspace is not None else 0
    L.check(plan._lib.tds_solve_batched(plan.handle, a.data_ptr(), b.data_ptr(), c.data_ptr(), d.data_ptr(),
                                        out.data_ptr(), wptr, wbytes, _stream_ptr(stream, dev)))
    return out


def solve_normalized(plan: Plan, a, c, d, out=None, workspace=None, stream=None):
    """tds_solve_normalized: the same solve for normalised systems (b = 1; no
    b array).  The plan needs k >= 1.  Returns x."""
    import torch
    info, need, want, dev = plan._solve_info()
    for name, t in (("a", a), ("c", c), ("d", d)):
        _check_fast(t, need, want, name, dev)
    if out is None:
        out = torch.empty_like(d)
    else:
        _check_fast(out, need, want, "out", dev)
    if workspace is None and info.workspace_bytes > 0:
        workspace = plan.workspace()
    wptr = workspace.data_ptr() if workspace is not None else None
    wbytes = workspace.numel() * workspace.element_size() if workspace is not None else 0
    L.check(plan._lib.tds_solve_normalized(plan.handle, a.data_ptr(), c.data_ptr(), d.data_ptr(), out.data_ptr(),
                                           wptr, wbytes, _stream_ptr(stream, dev)))
    return out


def split_slots(plan: Plan, a, b, c, d, workspace, stream=None):
    """tds_split_slots: run the split passes only; returns (a', c', d') as
    (num_slots, slot_rows) views into ``workspace`` (slot (s << k) + r = residue
    r of system s, normalised rows, Fig. 3a order)."""
    info, need, want, dev = plan._solve_info()
    for name, t in (("a", a), ("b", b), ("c", c), ("d", d)):
        _check_fast(t, need, want, name, dev)
    lay = plan.slots_layout()
    wbytes = workspace.numel() * workspace.element_size()
    L.check(plan._lib.tds_split_slots(plan.handle, a.data_ptr(), b.data_ptr(), c.data_ptr(), d.data_ptr(),
                                      workspace.data_ptr(), wbytes, _stream_ptr(stream, dev)))
    return slot_views(plan, workspace, lay)


def split_scatter(plan: Plan, a, b, c, d, dst, residues_per_group: int, first_pos: int, num_pos: int,
                  dst_stride: int, stream=None):
    """tds_split_scatter: the plan's one split pass with the all-to-all fused
    into its stores -- residue h q + rl of position first_pos + j goes to
    dst[t][h] + (rl * dst_stride + j) elements (t = a', c', d').  ``dst``: 3
    lists of device addresses (ints; peer-mapped addresses allowed) or
    tensors, one per destination."""
    info, need, want, dev = plan._solve_info()
    for name, t in (("a", a), ("b", b), ("c", c), ("d", d)):
        _check_fast(t, need, want, name, dev)
    spec = L.Scatter()
    groups = len(dst[0])
    spec.groups, spec.residues_per_group = groups, int(residues_per_group)
    spec.first_pos, spec.num_pos, spec.dst_stride = int(first_pos), int(num_pos), int(dst_stride)
    for t in range(3):
        if len(dst[t]) != groups:
            raise ValueError("dst: the same number of destinations for a', c', d'")
        for h, p in enumerate(dst[t]):
            spec.dst[t][h] = p if isinstance(p, int) else p.data_ptr()
    L.check(plan._lib.tds_split_scatter(plan.handle, a.data_ptr(), b.data_ptr(), c.data_ptr(), d.data_ptr(),
                                        ctypes.byref(spec), _stream_ptr(stream, dev)))


def solve_normalized_xscatter(plan: Plan, a, c, d, dst, rows_per_group: int, dst_system_stride: int,
                              workspace=None, stream=None):
    """tds_solve_normalized_xscatter: the normalised solve whose x placement
    writes rows [h rows_per_group, (h+1) rows_per_group) of every system
    straight to dst[h] + s * dst_system_stride (device / peer addresses or
    tensors)."""
    info, need, want, dev = plan._solve_info()
    for name, t in (("a", a), ("c", c), ("d", d)):
        _check_fast(t, need, want, name, dev)
    if workspace is None and info.workspace_bytes > 0:
        workspace = plan.workspace()
    spec = L.XScatter()
    spec.groups, spec.rows_per_group, spec.dst_system_stride = len(dst), int(rows_per_group), int(dst_system_stride)
    for h, p in enumerate(dst):
        spec.dst[h] = p if isinstance(p, int) else p.data_ptr()
    wptr = workspace.data_ptr() if workspace is not None else None
    wbytes = workspace.numel() * workspace.element_size() if workspace is not None else 0
    L.check(plan._lib.tds_solve_normalized_xscatter(plan.handle, a.data_ptr(), c.data_ptr(), d.data_ptr(),
                                                    ctypes.byref(spec), wptr, wbytes, _stream_ptr(stream, dev)))


def slot_views(plan: Plan, workspace, lay: Optional[dict] = None):
    """(a', c', d') views of the split slots inside ``workspace`` (no device work)."""
    info, _, want, _ = plan._solve_info()
    lay = lay or plan.slots_layout()
    typed = workspace.view(want)
    size = lay["num_slots"] * lay["slot_rows"]
    return tuple(typed[lay[k]:lay[k] + size].view(lay["num_slots"], lay["slot_rows"])
                 for k in ("a_offset", "c_offset", "d_offset"))


def unpack_residues(xs, x, n: int, m: int, k: int, slot_rows: int, batch_stride: int = 0, stream=None):
    """tds_unpack_residues: x[s*stride + r + 2^k j] = xs[((s << k) + r) * slot_rows + j]."""
    want = xs.dtype
    _check_fast(xs, (m << k) * slot_rows, want, "xs")
    stride = int(batch_stride) or int(n)
    _check_fast(x, (m - 1) * stride + n, want, "x")
    L.check(L.load().tds_unpack_residues(_dtype_code(want), int(n), int(m), int(k), int(slot_rows), xs.data_ptr(),
                                         x.data_ptr(), stride, _stream_ptr(stream, int(x.device.index))))
    return x


def generate_rows(n: int, row0: int, count: int, dtype="float32", seed: int = 1, mu: float = 1.0, device: int = 0,
                  out=None, stream=None):
    """tds_generate_rows: rows [row0, row0 + count) of one seeded system of n
    rows (identity rows outside [0, n)).  Returns (a, b, c, d), each (count,)."""
    import torch
    code = _dtype_code(dtype)
    tdt = torch.float32 if code == L.TDS_F32 else torch.float64
    if out is None:
        out = tuple(torch.empty(int(count), dtype=tdt, device=f"cuda:{device}") for _ in range(4))
    for name, t in zip("abcd", out):
        _check_fast(t, int(count), tdt, name)
    L.check(L.load().tds_generate_rows(code, int(n), int(row0), int(count), int(seed) & 0xFFFFFFFFFFFFFFFF,
                                       float(mu), *(t.data_ptr() for t in out),
                                       _stream_ptr(stream, int(out[0].device.index))))
    return out


def solve_interleaved(plan: Plan, a, b, c, d, out=None, workspace=None, stream=None):
    """tds_solve_interleaved: the same solve for arrays in the batch-interleaved
    layout (element i of system s at [i, s] of an (n, m) tensor).  Returns x, (n, m)."""
    import torch
    info, _, want, dev = plan._solve_info()
    need = info.n * info.m
    for name, t in (("a", a), ("b", b), ("c", c), ("d", d)):
        _check_fast(t, need, want, name, dev)
    if out is None:
        out = torch.empty_like(d)
    else:
        _check_fast(out, need, want, "out", dev)
    if workspace is None:
        workspace = torch.empty(plan.interleaved_workspace_bytes, dtype=torch.uint8, device=f"cuda:{dev}")
    wbytes = workspace.numel() * workspace.element_size()
    L.check(plan._lib.tds_solve_interleaved(plan.handle, a.data_ptr(), b.data_ptr(), c.data_ptr(), d.data_ptr(),
                                            out.data_ptr(), workspace.data_ptr(), wbytes,
                                            _stream_ptr(stream, dev)))
    return out


def solve_stages(plan: Plan, a, b, c, d, out, workspace, first: int, last: int, stream=None):
    """tds_solve_stages: run kernels first..last of the solve sequence (split
    passes 0..P-1, on-chip kernel P) -- for per-kernel timing."""
    info = plan.info_struct()
    for name, t in (("a", a), ("b", b), ("c", c), ("d", d), ("out", out)):
        _check_tensor(t, info, name)
    wptr = _ptr(workspace) if workspace is not None else None
    wbytes = workspace.numel() * workspace.element_size() if workspace is not None else 0
    L.check(plan._lib.tds_solve_stages(plan.handle, _ptr(a), _ptr(b), _ptr(c), _ptr(d), _ptr(out), wptr,
                                       wbytes, _stream_ptr(stream), int(first), int(last)))
    return out


def split_batched(plan: Plan, a, b, c, d, workspace=None, stream=None):
    """Diagnostic split stage (tds_split_batched): returns (a', c', d') (m, n)
    in canonical order, normalised so that b' = 1."""
    import torch
    info = plan.info_struct()
    for name, t in (("a", a), ("b", b), ("c", c), ("d", d)):
        _check_tensor(t, info, name)
    shape = (info.m, info.n)
    oa, oc, od = (torch.empty(shape, dtype=d.dtype, device=d.device) for _ in range(3))
    if workspace is None:
        workspace = plan.workspace()
    wptr = _ptr(workspace) if workspace is not None else None
    wbytes = workspace.numel() * workspace.element_size() if workspace is not None else 0
    L.check(plan._lib.tds_split_batched(plan.handle, _ptr(a), _ptr(b), _ptr(c), _ptr(d), _ptr(oa), _ptr(oc),
                                        _ptr(od), wptr, wbytes, _stream_ptr(stream)))
    return oa, oc, od


def generate(n: int, m: int, dtype="float32", seed: int = 1, first_system: int = 0, mu: float = 1.0,
             device: int = 0, batch_stride: int = 0, out=None, stream=None):
    """tds_generate: the seeded synthetic systems (inputs.py's "dd" family)
    drawn on the device.  Returns (a, b, c, d) as (m, batch_stride or n) CUDA
    tensors (or fills ``out``)."""
    import torch
    code = _dtype_code(dtype)
    stride = int(batch_stride) or int(n)
    tdt = torch.float32 if code == L.TDS_F32 else torch.float64
    if out is None:
        out = tuple(torch.empty((int(m), stride), dtype=tdt, device=f"cuda:{device}") for _ in range(4))
    for name, t in zip("abcd", out):
        _check_fast(t, (int(m) - 1) * stride + int(n), tdt, name)
    L.check(L.load().tds_generate(code, int(n), int(m), stride, int(seed) & 0xFFFFFFFFFFFFFFFF, int(first_system),
                                  float(mu), *(t.data_ptr() for t in out), _stream_ptr(stream, int(out[0].device.index))))
    return out


def version() -> int:
    return int(L.load().tds_version())
