"""ctypes mirror of include/jp.h (argument marshalling only).

Every entry point of libjp.so is exposed under its C name.  Structs are
declared field for field as in the header; the loader fails loudly when the
library has not been built -- there is no CPU fallback anywhere in this
package (every step of the loop runs in the CUDA kernels of libjp.so).
"""
from __future__ import annotations

import ctypes as C
import os
import threading

_HERE = os.path.dirname(os.path.abspath(__file__))
LIB_PATH = os.environ.get("JP_LIB") or os.path.join(_HERE, "libjp.so")

JP_OK, JP_ERR_ARG, JP_ERR_CUDA, JP_ERR_WORKSPACE, JP_ERR_ILLEGAL_MODE, JP_ERR_INDEX, JP_ERR_UNSUPPORTED = \
    0, -1, -2, -3, -4, -5, -6
STATUS_NAMES = {0: "JP_OK", -1: "JP_ERR_ARG", -2: "JP_ERR_CUDA", -3: "JP_ERR_WORKSPACE",
                -4: "JP_ERR_ILLEGAL_MODE", -5: "JP_ERR_INDEX", -6: "JP_ERR_UNSUPPORTED"}
JP_I32, JP_F32 = 0, 1
JP_OP_ADD_C, JP_OP_SAXPY, JP_OP_PRIV_TMP, JP_OP_STENCIL2 = 0, 1, 2, 3
JP_MODE_DOALL, JP_MODE_PRIVATIZED, JP_MODE_TLS, JP_MODE_SEQ_RECOMMENDED = 0, 1, 2, 3
MODE_NAMES = {0: "DOALL", 1: "PRIVATIZED", 2: "TLS", 3: "SEQ_RECOMMENDED"}
JP_SCHED_SHARING, JP_SCHED_STEALING, JP_SCHED_AUTO = 0, 1, 2
JP_MAX_LOOPS = 64
JP_TLS_RESTART, JP_TLS_ONCHIP = 0, 1
JP_WS_PROFILE, JP_WS_PRIV, JP_WS_TLS, JP_WS_SCHED, JP_WS_GUIDE, JP_WS_ALL = 1, 2, 4, 8, 16, 31
REGIONS = {"header": 0, "minW_A": 1, "minR_A": 2, "minW_T": 3, "minR_T": 4, "keys_A": 5, "keys_T": 6,
           "tls_S_A": 7, "tls_C_A": 8, "tls_C_T": 10, "sched": 11, "maxRx_A": 12, "guide": 13}


class jp_scalar(C.Union):
    _fields_ = [("i", C.c_int32), ("f", C.c_float)]


class jp_loop(C.Structure):
    _fields_ = [
        ("n", C.c_int64), ("iter_base", C.c_int64), ("ident_off", C.c_int64), ("op", C.c_int32), ("dtype", C.c_int32),
        ("r", C.c_void_p), ("r2", C.c_void_p), ("w", C.c_void_p), ("s", C.c_void_p),
        ("A", C.c_void_p), ("len_A", C.c_int64),
        ("X", C.c_void_p), ("len_X", C.c_int64),
        ("T", C.c_void_p), ("len_T", C.c_int64),
        ("c0", jp_scalar), ("c1", jp_scalar),
    ]


class jp_profile(C.Structure):
    _fields_ = [("n", C.c_int64), ("raw_iters", C.c_int64), ("war_iters", C.c_int64), ("waw_iters", C.c_int64),
                ("first_raw_iter", C.c_int64), ("d_raw", C.c_double), ("d_war", C.c_double),
                ("d_waw", C.c_double)]


class jp_tls_stats(C.Structure):
    _fields_ = [("committed", C.c_int64), ("executed", C.c_int64), ("windows", C.c_int64),
                ("violations", C.c_int64)]


class jp_tls_cfg(C.Structure):
    _fields_ = [("window", C.c_int64), ("w_max", C.c_int64), ("path", C.c_int32), ("cluster", C.c_int32),
                ("guided", C.c_int32), ("recovery", C.c_int32)]


class jp_sched_cfg(C.Structure):
    _fields_ = [("scheme", C.c_int32), ("tls_path", C.c_int32), ("tau_high", C.c_double),
                ("chunk_iters", C.c_int64), ("tls_window", C.c_int64), ("tls_w_max", C.c_int64),
                ("tls_recovery", C.c_int32), ("static_check", C.c_int32)]


class jp_static(C.Structure):
    _fields_ = [("affine", C.c_int32), ("independent", C.c_int32), ("in_range", C.c_int32), ("reserved", C.c_int32),
                ("alpha", C.c_int64 * 4), ("beta", C.c_int64 * 4)]


class jp_workflow_plan(C.Structure):
    _fields_ = [("scheme", C.c_int32), ("n_batches", C.c_int32), ("batch", C.c_int32 * 64), ("deps", C.c_uint64 * 64)]


class jp_sched_result(C.Structure):
    _fields_ = [("mode", C.c_int32), ("profiled", C.c_int32), ("prof", jp_profile), ("tls", jp_tls_stats),
                ("n_tasks", C.c_int64), ("n_batches", C.c_int64), ("task_mode_iters", C.c_int64 * 4),
                ("tls_w_max", C.c_int64), ("tls_path", C.c_int32), ("tls_guided", C.c_int32),
                ("tls_recovery", C.c_int32), ("tls_cluster", C.c_int32)]


# (name, restype, argtypes) -- one line per declaration of include/jp.h
_P, _V, _I32, _I64, _SZ, _D = C.POINTER, C.c_void_p, C.c_int32, C.c_int64, C.c_size_t, C.c_double
SIGNATURES = [
    ("jp_workspace_bytes", _SZ, [_P(jp_loop), _I32]),
    ("jp_ws_region", _I32, [_P(jp_loop), _I32, _P(_SZ), _P(_SZ)]),
    ("jp_validate", _I32, [_P(jp_loop), _V, _SZ, _P(_I64), _V]),
    ("jp_profile_stamp", _I32, [_P(jp_loop), _V, _SZ, _V]),
    ("jp_profile_classify", _I32, [_P(jp_loop), _V, _SZ, _V, _I64, _V, _P(jp_profile), _V]),
    ("jp_profile_density", _I32, [_P(jp_loop), _V, _SZ, _V, _I64, _V, _P(jp_profile), _V]),
    ("jp_select_mode", _I32, [_P(jp_loop), _P(jp_profile), _D]),
    ("jp_static_check", _I32, [_P(jp_loop), _V, _SZ, _P(jp_static), _V]),
    ("jp_affine_dependence", _I32, [_I64, _I64, _I64, _I64, _I64]),
    ("jp_run_doall", _I32, [_P(jp_loop), _P(jp_profile), _V, _SZ, _V]),
    ("jp_run_privatized", _I32, [_P(jp_loop), _P(jp_profile), _V, _SZ, _V]),
    ("jp_priv_stream", _I32, [_P(jp_loop), _P(jp_profile), _V, _SZ, _I32, _V]),
    ("jp_priv_finalize", _I32, [_P(jp_loop), _V, _SZ, _V]),
    ("jp_doall_kernel", _I32, [_I32]),
    ("jp_tls_guide", _I32, [_P(jp_loop), _V, _SZ, _V]),
    ("jp_tls_next_window", _I64, [_I64, _I64, _I64, _I64]),
    ("jp_run_tls", _I32, [_P(jp_loop), _P(jp_tls_cfg), _P(jp_profile), _V, _SZ, _P(jp_tls_stats), _V]),
    ("jp_schedule", _I32, [_P(jp_loop), _P(jp_sched_cfg), _V, _SZ, _P(jp_sched_result), _V]),
    ("jp_stage_bytes", _SZ, [_P(jp_loop)]),
    ("jp_schedule_host", _I32, [_P(jp_loop), _P(jp_sched_cfg), _V, _SZ, _V, _SZ, _P(jp_sched_result), _V]),
    ("jp_plan_sharing", _I32, [_I64, _I32, _P(_D), _P(_I64)]),
    ("jp_plan_stealing", _I32, [_P(_I64), _I64, _I32, _I64, _P(_D), _D, _P(_I64), _I64, _P(_I64), _P(_I64)]),
    ("jp_plan_workflow", _I32, [_P(jp_loop), _I32, _I32, _P(jp_workflow_plan)]),
    ("jp_schedule_workflow", _I32, [_P(jp_loop), _I32, _P(jp_sched_cfg), _P(_V), _P(_SZ), _P(jp_sched_result),
                                    _P(jp_workflow_plan), _V]),
    ("jp_merge_apply", _I32, [_V, _I64, _V, _V]),
    ("jp_plan", _I32, [_P(jp_loop), _P(jp_sched_cfg), _P(jp_profile), _I64, _I32, _P(_D), _P(_I64), _I64, _P(_I64)]),
    ("jp_plan_tasks", _I32, [_P(jp_loop), _P(_I64), _I64, _D, _V, _SZ, _P(_I64), _P(_I32), _P(C.c_uint64), _V]),
    ("jp_profile_plan_tasks", _I32, [_P(jp_loop), _I64, _D, _V, _SZ, _P(jp_profile), _P(_I64), _P(_I64), _P(_I32),
                                     _P(C.c_uint64), _V]),
    ("jp_export_keys", _I32, [_P(jp_loop), _V, _SZ, _V]),
    ("jp_run_priv_claim", _I32, [_P(jp_loop), _V, _P(_I64), _I32, _I32, _V, _V, _V, _SZ, _I32, _V]),
    ("jp_keys_merge_p2p", _I32, [_P(_V), _I32, _V, _I64, _V, _I64, _V, _V, _V]),
    ("jp_priv_inbox_bytes", _SZ, [_P(jp_loop), _I32]),
    ("jp_priv_stream_merge", _I32, [_P(jp_loop), _P(jp_profile), _V, _SZ, _P(_V), _I32, _I32, _V, _V]),
    ("jp_run_doall_spill", _I32, [_P(jp_loop), _I32, _I32, _I64, _V, _V, _I32, _V]),
    ("jp_ipc_export", _I32, [_V, _V, _P(_I64)]),
    ("jp_ipc_import", _I32, [_V, _I64, _P(_V)]),
    ("jp_ipc_close", _I32, [_V, _I64]),
    ("jp_sparse_scratch_bytes", _SZ, [_I64, _I32]),
    ("jp_sparse_pack", _I32, [_V, _V, _I32, _I64, _I64, _I64, _I64, _I32, _V, _I64, _P(_I64), _V, _SZ, _V]),
    ("jp_sparse_reduce_max", _I32, [_V, _V, _I32, _I64, _V, _I64, _V]),
    ("jp_sparse_gather", _I32, [_V, _V, _I32, _I64, _V, _I64, _V]),
    ("jp_sparse_scatter", _I32, [_V, _V, _I32, _I64, _V, _I64, _V]),
    ("jp_last_error", C.c_char_p, []),
    ("jp_version", C.c_char_p, []),
    ("jp_launch_count", _I64, []),
    ("jp_tls_grid_window", _I64, []),
]

# reading A4's Fig. 2(b) threshold, the library's default (jp_host.h kTauHigh, measured)
TAU_HIGH = 0.999

_lock = threading.Lock()
_lib = None


class JPError(RuntimeError):
    def __init__(self, status: int, msg: str):
        super().__init__(f"{STATUS_NAMES.get(status, status)}: {msg}")
        self.status = status


def lib():
    """Load libjp.so (once).  Raises if it was not built: no fallback exists."""
    global _lib
    with _lock:
        if _lib is None:
            if not os.path.exists(LIB_PATH):
                raise ImportError(f"{LIB_PATH} is missing: build it with `python -c 'import __graft_entry__ as g; "
                                  "g.build()'` (the CUDA library is the only implementation)")
            L = C.CDLL(LIB_PATH)
            for name, res, args in SIGNATURES:
                f = getattr(L, name)
                f.restype = res
                f.argtypes = args
            _lib = L
    return _lib


def check(status: int):
    if status != JP_OK:
        raise JPError(status, lib().jp_last_error().decode())
    return status
