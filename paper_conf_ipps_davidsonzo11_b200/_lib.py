"""ctypes declarations for libtds.so (include/tds.h).  Argument marshalling only.

The library is loaded lazily; a missing library raises (there is no fallback).
"""
from __future__ import annotations

import ctypes
import os

_HERE = os.path.dirname(os.path.abspath(__file__))
LIB_PATH = os.path.join(_HERE, "libtds.so")

TDS_OK = 0
TDS_F32, TDS_F64 = 0, 1
TDS_PARAMS_DEFAULT, TDS_PARAMS_STATIC, TDS_PARAMS_TUNED = 0, 1, 2
TDS_MAX_PASSES = 8

STATUS_NAMES = {
    0: "TDS_OK", 1: "TDS_ERR_INVALID_ARG", 2: "TDS_ERR_UNSUPPORTED", 3: "TDS_ERR_NO_MEMORY",
    4: "TDS_ERR_WORKSPACE", 5: "TDS_ERR_CUDA", 6: "TDS_ERR_TUNE", 7: "TDS_ERR_DEVICE_MISMATCH",
}

# Every symbol include/tds.h declares (checked by tests/test_abi.py).
EXPORTED = (
    "tds_plan", "tds_plan_from_props", "tds_device_props_query", "tds_plan_info_get",
    "tds_plan_set_params", "tds_plan_permutation", "tds_plan_destroy", "tds_tune",
    "tds_plan_tune_trials", "tds_solve_batched", "tds_solve_stages", "tds_split_batched", "tds_status_string",
    "tds_interleaved_workspace_bytes", "tds_solve_interleaved",
    "tds_last_error", "tds_version", "tds_tune_search", "tds_generate", "tds_generate_rows",
    "tds_solve_normalized", "tds_plan_slots_layout", "tds_split_slots", "tds_unpack_residues",
    "tds_split_scatter", "tds_solve_normalized_xscatter",
)


class DeviceProps(ctypes.Structure):
    _fields_ = [("sm_count", ctypes.c_int32), ("smem_optin_bytes", ctypes.c_int32),
                ("smem_per_sm_bytes", ctypes.c_int32), ("regs_per_sm", ctypes.c_int32),
                ("max_threads_per_block", ctypes.c_int32), ("warp_size", ctypes.c_int32),
                ("cc_major", ctypes.c_int32), ("cc_minor", ctypes.c_int32),
                ("l2_bytes", ctypes.c_int64), ("global_mem_bytes", ctypes.c_int64)]


class Params(ctypes.Structure):
    _fields_ = [("k", ctypes.c_int32), ("passes", ctypes.c_int32),
                ("k_pass", ctypes.c_int32 * TDS_MAX_PASSES), ("cr_levels", ctypes.c_int32),
                ("thomas_chains", ctypes.c_int32), ("cluster", ctypes.c_int32),
                ("tl_levels", ctypes.c_int32),
                ("split_tile_rows", ctypes.c_int32),
                ("split_threads", ctypes.c_int32), ("theta", ctypes.c_int32),
                ("chunk_systems", ctypes.c_int32), ("split_only", ctypes.c_int32),
                ("x_group", ctypes.c_int32), ("strided", ctypes.c_int32)]


class PlanInfo(ctypes.Structure):
    _fields_ = [("dtype", ctypes.c_int32), ("mode", ctypes.c_int32), ("tuned", ctypes.c_int32),
                ("device", ctypes.c_int32), ("n", ctypes.c_int64), ("m", ctypes.c_int64),
                ("batch_stride", ctypes.c_int64), ("params", Params), ("n_sub", ctypes.c_int64),
                ("num_subsystems", ctypes.c_int64), ("n_sub_target", ctypes.c_int32),
                ("n_onchip_max", ctypes.c_int32), ("split_kp_max", ctypes.c_int32),
                ("onchip_threads", ctypes.c_int32), ("subsys_per_cta", ctypes.c_int32),
                ("split_segments", ctypes.c_int32), ("split_tile_eff", ctypes.c_int32),
                ("chunks", ctypes.c_int32), ("launches", ctypes.c_int32),
                ("slot_rows", ctypes.c_int64), ("workspace_bytes", ctypes.c_size_t),
                ("onchip_form", ctypes.c_int32)]


class SlotsLayout(ctypes.Structure):
    _fields_ = [("a_offset", ctypes.c_int64), ("c_offset", ctypes.c_int64), ("d_offset", ctypes.c_int64),
                ("slot_rows", ctypes.c_int64), ("num_slots", ctypes.c_int64)]


class Scatter(ctypes.Structure):
    _fields_ = [("groups", ctypes.c_int32), ("residues_per_group", ctypes.c_int32),
                ("first_pos", ctypes.c_int64), ("num_pos", ctypes.c_int64), ("dst_stride", ctypes.c_int64),
                ("dst", (ctypes.c_void_p * 8) * 3)]


class XScatter(ctypes.Structure):
    _fields_ = [("groups", ctypes.c_int32), ("rows_per_group", ctypes.c_int64),
                ("dst_system_stride", ctypes.c_int64), ("dst", ctypes.c_void_p * 8)]


# tds_tune_search's cost callback: double (*)(const tds_params *, void *)
COST_FN = ctypes.CFUNCTYPE(ctypes.c_double, ctypes.POINTER(Params), ctypes.c_void_p)

_lib = None


def load() -> ctypes.CDLL:
    """Load libtds.so (build it with ``python -c 'import __graft_entry__ as g; g.build()'``)."""
    global _lib
    if _lib is not None:
        return _lib
    if not os.path.exists(LIB_PATH):
        raise RuntimeError(f"libtds.so not found at {LIB_PATH}: the CUDA extension is not built "
                           "(run __graft_entry__.build()); there is no CPU fallback")
    lib = ctypes.CDLL(LIB_PATH)
    P, I64, I32, VP, SZ = ctypes.c_void_p, ctypes.c_int64, ctypes.c_int, ctypes.c_void_p, ctypes.c_size_t
    PP = ctypes.POINTER(ctypes.c_void_p)
    sig = {
        "tds_plan": (I32, [PP, I32, I32, I64, I64, I64, I32]),
        "tds_plan_from_props": (I32, [PP, ctypes.POINTER(DeviceProps), I32, I64, I64, I64, I32]),
        "tds_device_props_query": (I32, [I32, ctypes.POINTER(DeviceProps)]),
        "tds_plan_info_get": (I32, [P, ctypes.POINTER(PlanInfo)]),
        "tds_plan_set_params": (I32, [P, ctypes.POINTER(Params)]),
        "tds_plan_permutation": (I32, [P, VP, I64]),
        "tds_plan_destroy": (I32, [P]),
        "tds_tune": (I32, [P, VP, ctypes.c_char_p]),
        "tds_plan_tune_trials": (I32, [P, ctypes.POINTER(ctypes.c_int32)]),
        "tds_solve_batched": (I32, [P, VP, VP, VP, VP, VP, VP, SZ, VP]),
        "tds_solve_stages": (I32, [P, VP, VP, VP, VP, VP, VP, SZ, VP, ctypes.c_int32, ctypes.c_int32]),
        "tds_split_batched": (I32, [P, VP, VP, VP, VP, VP, VP, VP, VP, SZ, VP]),
        "tds_interleaved_workspace_bytes": (I32, [P, ctypes.POINTER(ctypes.c_size_t)]),
        "tds_solve_interleaved": (I32, [P, VP, VP, VP, VP, VP, VP, SZ, VP]),
        "tds_tune_search": (I32, [P, COST_FN, VP, ctypes.c_char_p]),
        "tds_generate": (I32, [I32, I64, I64, I64, ctypes.c_uint64, I64, ctypes.c_double, VP, VP, VP, VP, VP]),
        "tds_generate_rows": (I32, [I32, I64, I64, I64, ctypes.c_uint64, ctypes.c_double, VP, VP, VP, VP, VP]),
        "tds_solve_normalized": (I32, [P, VP, VP, VP, VP, VP, SZ, VP]),
        "tds_plan_slots_layout": (I32, [P, ctypes.POINTER(SlotsLayout)]),
        "tds_split_slots": (I32, [P, VP, VP, VP, VP, VP, SZ, VP]),
        "tds_unpack_residues": (I32, [I32, I64, I64, I32, I64, VP, VP, I64, VP]),
        "tds_split_scatter": (I32, [P, VP, VP, VP, VP, ctypes.POINTER(Scatter), VP]),
        "tds_solve_normalized_xscatter": (I32, [P, VP, VP, VP, ctypes.POINTER(XScatter), VP, SZ, VP]),
        "tds_status_string": (ctypes.c_char_p, [I32]),
        "tds_last_error": (ctypes.c_char_p, []),
        "tds_version": (I32, []),
    }
    for name, (res, args) in sig.items():
        fn = getattr(lib, name)
        fn.restype = res
        fn.argtypes = args
    _lib = lib
    return lib


class TdsError(RuntimeError):
    def __init__(self, status: int, detail: str = ""):
        self.status = status
        self.name = STATUS_NAMES.get(status, str(status))
        super().__init__(f"{self.name}: {detail}" if detail else self.name)


def check(status: int) -> None:
    if status != TDS_OK:
        lib = load()
        raise TdsError(status, lib.tds_last_error().decode(errors="replace"))
