"""ctypes binding of libswdual.so (include/swdual.h).  Argument marshalling only:
every step of the path runs in the library's CUDA kernels.  There is no CPU
fallback: if the shared library is missing this module raises on import of the
first call."""
from __future__ import annotations

import ctypes
import os

_HERE = os.path.dirname(os.path.abspath(__file__))
# SWDUAL_LIB overrides the in-tree library (A/B experiments with alternative builds)
LIB_PATH = os.environ.get("SWDUAL_LIB") or os.path.join(_HERE, "libswdual.so")

SW_OK, SW_EINVAL, SW_ENOMEM, SW_ECUDA, SW_ESTATE, SW_EUNSUPPORTED = 0, -1, -2, -3, -4, -5
SW_FLAG_TIMING = 1

EXPORTS = ["sw_init", "sw_load_db", "sw_search", "sw_free_db", "sw_free", "sw_last_error",
           "sw_db_info", "sw_last_stats", "sw_set_option", "sw_encode_ascii", "sw_schedule_dual", "sw_align",
           "sw_encode_nucleotide", "sw_search_cpu", "sw_schedule_dual_dp", "sw_load_db_mapped",
           "sw_assembly_create", "sw_assemble", "sw_assembly_free", "sw_subset_host"]


class SWError(RuntimeError):
    def __init__(self, code: int, msg: str):
        super().__init__(f"swdual error {code}: {msg}")
        self.code = code


class DbInfo(ctypes.Structure):
    _fields_ = [("n_seqs", ctypes.c_int64), ("n_residues", ctypes.c_int64), ("n_pairs", ctypes.c_int64),
                ("n_long_pairs", ctypes.c_int64), ("max_len", ctypes.c_int64),
                ("alphabet_size", ctypes.c_int32), ("device", ctypes.c_int32)]


class Block(ctypes.Structure):
    _fields_ = [("src_off", ctypes.c_int64), ("row_off", ctypes.c_int64), ("col_off", ctypes.c_int64),
                ("n_rows", ctypes.c_int64), ("n_cols", ctypes.c_int64)]


class Stats(ctypes.Structure):
    _fields_ = [("cells", ctypes.c_double), ("cells_short", ctypes.c_double), ("cells_computed", ctypes.c_double),
                ("short_ms", ctypes.c_double), ("long_ms", ctypes.c_double), ("search_ms", ctypes.c_double),
                ("n_launches", ctypes.c_int32), ("n_score_launches", ctypes.c_int32),
                ("n_overflow", ctypes.c_int32), ("timing_valid", ctypes.c_int32),
                ("last_G", ctypes.c_int32), ("last_R", ctypes.c_int32)]


_lib = None


def lib() -> ctypes.CDLL:
    global _lib
    if _lib is not None:
        return _lib
    if not os.path.exists(LIB_PATH):
        raise ImportError(f"{LIB_PATH} is missing: run `make` (or __graft_entry__.build()) first; "
                          "there is no fallback implementation")
    L = ctypes.CDLL(LIB_PATH)
    V, I32, I64, U32, P = ctypes.c_void_p, ctypes.c_int32, ctypes.c_int64, ctypes.c_uint32, ctypes.POINTER
    L.sw_init.restype = I32
    L.sw_init.argtypes = [I32, U32, P(V)]
    L.sw_load_db.restype = I32
    L.sw_load_db.argtypes = [V, V, V, I64, I32, V, P(V)]
    L.sw_search.restype = I32
    L.sw_search.argtypes = [V, V, V, I32, V, V, I32, I32, V, V]
    L.sw_free_db.restype = I32
    L.sw_free_db.argtypes = [V]
    L.sw_free.restype = I32
    L.sw_free.argtypes = [V]
    L.sw_last_error.restype = ctypes.c_char_p
    L.sw_last_error.argtypes = [V]
    L.sw_db_info.restype = I32
    L.sw_db_info.argtypes = [V, P(DbInfo)]
    L.sw_last_stats.restype = I32
    L.sw_last_stats.argtypes = [V, P(Stats)]
    L.sw_set_option.restype = I32
    L.sw_set_option.argtypes = [V, ctypes.c_char_p, I64]
    L.sw_encode_ascii.restype = I32
    L.sw_encode_ascii.argtypes = [ctypes.c_char_p, I64, V]
    L.sw_schedule_dual.restype = I32
    L.sw_schedule_dual.argtypes = [I64, V, V, I32, I32, V, P(ctypes.c_double), P(ctypes.c_double)]
    L.sw_encode_nucleotide.restype = I32
    L.sw_encode_nucleotide.argtypes = [ctypes.c_char_p, I64, V]
    L.sw_load_db_mapped.restype = I32
    L.sw_load_db_mapped.argtypes = [V, V, V, I64, I32, V, I64, V, P(V)]
    L.sw_schedule_dual_dp.restype = I32
    L.sw_schedule_dual_dp.argtypes = [I64, V, V, I32, I32, V, P(ctypes.c_double), P(ctypes.c_double)]
    L.sw_search_cpu.restype = I32
    L.sw_search_cpu.argtypes = [V, V, I32, V, V, I64, I32, V, I32, I32, I32, V]
    L.sw_align.restype = I32
    L.sw_align.argtypes = [V, V, V, I32, V, V, I32, V, I32, I32, V, V, V, V, V]
    L.sw_assembly_create.restype = I32
    L.sw_assembly_create.argtypes = [V, V, I32, V, I64, V, I64, I32, I64, P(V)]
    L.sw_assemble.restype = I32
    L.sw_assemble.argtypes = [V, V, I64, V, V]
    L.sw_subset_host.restype = I32
    L.sw_subset_host.argtypes = [V, V, I64, V, I64, V, V, P(I64)]
    L.sw_assembly_free.restype = I32
    L.sw_assembly_free.argtypes = [V]
    _lib = L
    return L


def check(rc: int, handle=None) -> None:
    if rc != SW_OK:
        msg = lib().sw_last_error(handle)
        raise SWError(rc, msg.decode() if msg else "")
