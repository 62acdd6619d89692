"""ctypes loader for libaol.so (the C ABI of include/aol.h).

Argument marshalling only.  There is NO fallback: if the CUDA library is
missing or fails to load, every entry point raises.
"""
from __future__ import annotations

import ctypes
import os

_HERE = os.path.dirname(os.path.abspath(__file__))
# AOL_LIB_PATH lets tools load an instrumented build of the SAME library (e.g. tools/stream_probe.sh);
# it is never a fallback: the path must hold a libaol.so built from csrc/.
LIB_PATH = os.environ.get("AOL_LIB_PATH") or os.path.join(_HERE, "libaol.so")

MAX_RANK = 8

# aol_status_t
OK, E_INVALID, E_SHAPE, E_DTYPE, E_ALIGN, E_WORKSPACE, E_RANGE, E_CUDA = 0, -1, -2, -3, -4, -5, -6, -7
STATUS_NAMES = {0: "AOL_OK", -1: "AOL_E_INVALID", -2: "AOL_E_SHAPE", -3: "AOL_E_DTYPE", -4: "AOL_E_ALIGN",
                -5: "AOL_E_WORKSPACE", -6: "AOL_E_RANGE", -7: "AOL_E_CUDA"}
# aol_dtype_t
U8, I16, I32, I64, RAW8, RAW16, RAW32, RAW64 = 1, 2, 3, 4, 5, 6, 7, 8
RGB8 = 9   # packed 24-bit pixels [frames][H][W][3] (fused downscaler input only)
# aol_scatter_mode_t
SCATTER_FAST, SCATTER_SEQUENTIAL = 0, 1
# aol_preset_t
PRESET_H_IN, PRESET_H_OUT, PRESET_V_IN, PRESET_V_OUT = 0, 1, 2, 3


class AolError(RuntimeError):
    def __init__(self, status: int, message: str):
        super().__init__(f"{STATUS_NAMES.get(status, status)}: {message}")
        self.status = status


class aol_tiler_t(ctypes.Structure):
    _fields_ = [
        ("array_rank", ctypes.c_int32),
        ("rep_rank", ctypes.c_int32),
        ("pattern_rank", ctypes.c_int32),
        ("array_shape", ctypes.c_int64 * MAX_RANK),
        ("rep_shape", ctypes.c_int64 * MAX_RANK),
        ("pattern_shape", ctypes.c_int64 * MAX_RANK),
        ("origin", ctypes.c_int64 * MAX_RANK),
        ("paving", (ctypes.c_int64 * MAX_RANK) * MAX_RANK),
        ("fitting", (ctypes.c_int64 * MAX_RANK) * MAX_RANK),
    ]


MAX_FILTER_PATTERN, MAX_WINDOWS = 64, 16
FILTER_H, FILTER_V = 0, 1


class aol_filter_t(ctypes.Structure):
    _fields_ = [("in_", aol_tiler_t), ("out", aol_tiler_t), ("n_windows", ctypes.c_int32),
                ("window_len", ctypes.c_int32), ("divisor", ctypes.c_int32),
                ("window_start", ctypes.c_int32 * MAX_WINDOWS)]


# aol_launch_opts_t.flags bits (include/aol_tuning.h AOL_FLAG_*; A/B experiments, results are identical)
FLAG_U8_ONE_REP, FLAG_NO_PDL, FLAG_I32_LINEAR = 32, 64, 128
FLAG_ROW_STAGES, FLAG_TRIPLE_STAGES, FLAG_I32_STRIPS = 512, 1024, 2048
FLAGS = {"U8_ONE_REP": FLAG_U8_ONE_REP, "NO_PDL": FLAG_NO_PDL, "I32_LINEAR": FLAG_I32_LINEAR,
         "ROW_STAGES": FLAG_ROW_STAGES, "TRIPLE_STAGES": FLAG_TRIPLE_STAGES, "I32_STRIPS": FLAG_I32_STRIPS}


class aol_launch_opts_t(ctypes.Structure):
    _fields_ = [("ctas_per_sm", ctypes.c_int32), ("stages", ctypes.c_int32),
                ("bands_per_unit", ctypes.c_int32), ("kernel", ctypes.c_int32),
                ("flags", ctypes.c_int32)]


class aol_plan_t(ctypes.Structure):
    _fields_ = [("kernel", ctypes.c_int32), ("grid", ctypes.c_int32), ("block", ctypes.c_int32),
                ("smem_bytes", ctypes.c_int32), ("stages", ctypes.c_int32), ("bands_per_unit", ctypes.c_int32),
                ("units", ctypes.c_int64), ("ctas_per_sm", ctypes.c_int32), ("num_sms", ctypes.c_int32)]


_P = ctypes.c_void_p
_I64 = ctypes.c_int64
_I32 = ctypes.c_int32
_ST = ctypes.c_int  # aol_status_t
_TP = ctypes.POINTER(aol_tiler_t)
_FP = ctypes.POINTER(aol_filter_t)

SIGNATURES = {
    "aol_version": ([], ctypes.c_int),
    "aol_last_error": ([], ctypes.c_char_p),
    "aol_tiler_preset": ([ctypes.c_int, _I64, _I64, _TP], _ST),
    "aol_tiler_validate": ([_TP], _ST),
    "aol_tiler_is_injective": ([_TP, ctypes.POINTER(ctypes.c_int)], _ST),
    "aol_tiler_gather": ([_TP, ctypes.c_int, _P, _P, _P], _ST),
    "aol_tiler_scatter_workspace_bytes": ([_TP], ctypes.c_size_t),
    "aol_tiler_scatter": ([_TP, ctypes.c_int, _P, _P, ctypes.c_int, _P, ctypes.c_size_t, _P], _ST),
    "aol_downscale_h": ([_P, _P, _I64, _I64, _I64, _P], _ST),
    "aol_downscale_v": ([_P, _P, _I64, _I64, _I64, _P], _ST),
    "aol_downscale_frame": ([_P, ctypes.c_int, _P, _I64, _I64, _I64, _I64, _P, _P], _ST),
    "aol_downscale_frame_ex": ([_P, ctypes.c_int, _P, _I64, _I64, _I64, _I64, _P,
                                ctypes.POINTER(aol_launch_opts_t), _P], _ST),
    "aol_downscale_frame_plan": ([ctypes.c_int, _I64, _I64, _I64, _I64, ctypes.POINTER(aol_launch_opts_t),
                                  ctypes.POINTER(aol_plan_t)], _ST),
    "aol_downscale_frame_out": ([_P, ctypes.c_int, _P, ctypes.c_int, _I64, _I64, _I64, _I64, _P,
                                 ctypes.POINTER(aol_launch_opts_t), _P], _ST),
    "aol_downscale_frame_plan_out": ([ctypes.c_int, ctypes.c_int, _I64, _I64, _I64, _I64,
                                      ctypes.POINTER(aol_launch_opts_t), ctypes.POINTER(aol_plan_t)], _ST),
    "aol_frame_checksum": ([_P, _I64, _I64, _I64, _I64, _P, _P], _ST),
    "aol_downscale_frame_host_workspace_bytes": ([ctypes.c_int, _I64, _I64, _I64, _I64], ctypes.c_size_t),
    "aol_downscale_frame_host": ([_P, ctypes.c_int, _P, _I64, _I64, _I64, _I64, _P, _I64, _P, ctypes.c_size_t,
                                  _P, _P, _P], _ST),
    "aol_filter_preset": ([ctypes.c_int, _I64, _I64, _I64, _FP], _ST),
    "aol_filter_validate": ([_FP], _ST),
    "aol_filter_apply": ([_FP, _P, _P, _P], _ST),
    "aol_filter_chain_apply": ([_FP, _FP, _P, _P, _P, ctypes.c_size_t, _P], _ST),
    "aol_debug_fail_next_launches": ([ctypes.c_int], None),
    "aol_debug_last_kernel": ([], ctypes.c_char_p),
    "aol_debug_set_chain_jit": ([ctypes.c_int], None),
    "aol_debug_sep_jit_compile": ([_FP, _FP, ctypes.c_char_p, ctypes.c_size_t], ctypes.c_int),
    "aol_frame_plan_create": ([_P, ctypes.c_int, _P, ctypes.c_int, _I64, _I64, _I64, _I64,
                               ctypes.POINTER(aol_launch_opts_t), ctypes.POINTER(_P)], _ST),
    "aol_frame_plan_launch": ([_P, _P, _P], _ST),
    "aol_frame_plan_info": ([_P, ctypes.POINTER(aol_plan_t)], _ST),
    "aol_frame_plan_destroy": ([_P], _ST),
    "aol_synth_frames": ([ctypes.c_uint64, _I64, _I64, _I64, _I64, _I64, _I32, _I32, ctypes.c_int, _P, _P], _ST),
}

_lib = None


def lib() -> ctypes.CDLL:
    """Load libaol.so (raises if it was never built -- there is no fallback path)."""
    global _lib
    if _lib is None:
        if not os.path.exists(LIB_PATH):
            raise ImportError(f"{LIB_PATH} not found: build it with `make` or __graft_entry__.build() "
                              "(the CUDA library is required; there is no CPU fallback)")
        L = ctypes.CDLL(LIB_PATH)
        for name, (args, res) in SIGNATURES.items():
            f = getattr(L, name, None)
            if f is None:
                # only an older build loaded through AOL_LIB_PATH for an A/B can lack a symbol (the in-tree
                # library exports every one: tests/test_abi.py); its callers then fail when they use it
                if LIB_PATH != os.path.join(_HERE, "libaol.so"):
                    continue
                raise ImportError(f"{LIB_PATH} lacks {name}: rebuild it (make)")
            f.argtypes = args
            f.restype = res
        _lib = L
    return _lib


def check(status: int) -> None:
    if status != OK:
        msg = lib().aol_last_error()
        raise AolError(status, msg.decode() if msg else "")
