"""Python API over the C ABI (include/swdual.h): same names, marshalling only.

    h  = Handle(device=0)
    db = h.load_db(codes, offsets, alphabet_size=24)        # sw_load_db
    S  = h.search(q_codes, q_offsets, db, blosum62(), 10, 2) # sw_search -> int32[Q, N]

PyTorch supplies device memory (output tensors) and streams; every score is
computed by the library's CUDA kernels.
"""
from __future__ import annotations

import ctypes

import numpy as np

from ._lib import Block, DbInfo, Stats, SW_FLAG_TIMING, check, lib

try:  # torch is plumbing only (device buffers, streams)
    import torch
except Exception:  # pragma: no cover
    torch = None


def _host(a, dtype) -> np.ndarray:
    if torch is not None and isinstance(a, torch.Tensor):
        a = a.detach().cpu().numpy()
    return np.ascontiguousarray(np.asarray(a, dtype=dtype))


def _vp(a: np.ndarray):
    return a.ctypes.data_as(ctypes.c_void_p)


def _stream_ptr(stream):
    if stream is None:
        if torch is not None and torch.cuda.is_available():
            return ctypes.c_void_p(torch.cuda.current_stream().cuda_stream)
        return ctypes.c_void_p(0)
    if torch is not None and isinstance(stream, torch.cuda.Stream):
        return ctypes.c_void_p(stream.cuda_stream)
    return ctypes.c_void_p(int(stream))


class Database:
    """A packed, device-resident database (sw_db_t)."""

    def __init__(self, handle: "Handle", ptr: ctypes.c_void_p, n_seqs: int):
        self.handle = handle
        self.ptr = ptr
        self.n_seqs = n_seqs

    def info(self) -> dict:
        out = DbInfo()
        check(lib().sw_db_info(self.ptr, ctypes.byref(out)), self.handle.ptr)
        return {f: getattr(out, f) for f, _ in DbInfo._fields_}

    def free(self) -> None:
        if self.ptr:
            lib().sw_free_db(self.ptr)
            self.ptr = None


class Assembly:
    """sw_assembly_t: the fixed block layout of a multi-GPU placement."""

    def __init__(self, handle: "Handle", ptr: ctypes.c_void_p):
        self.handle = handle
        self.ptr = ptr

    def __call__(self, src, out, stream=None) -> None:
        """sw_assemble: device src (gathered int32 blocks) -> device out [Q][N], stream-ordered."""
        if not (torch is not None and isinstance(src, torch.Tensor) and isinstance(out, torch.Tensor)
                and src.is_cuda and out.is_cuda and src.dtype == torch.int32 and out.dtype == torch.int32
                and src.is_contiguous() and out.is_contiguous()):
            raise ValueError("assemble: src and out must be contiguous int32 CUDA tensors")
        check(lib().sw_assemble(self.ptr, ctypes.c_void_p(src.data_ptr()), src.numel(),
                                ctypes.c_void_p(out.data_ptr()), _stream_ptr(stream)), self.handle.ptr)

    def free(self) -> None:
        if self.ptr:
            lib().sw_assembly_free(self.ptr)
            self.ptr = None


class Handle:
    """sw_handle_t bound to one CUDA device."""

    def __init__(self, device: int = 0, timing: bool = False):
        self.ptr = ctypes.c_void_p()
        check(lib().sw_init(int(device), SW_FLAG_TIMING if timing else 0, ctypes.byref(self.ptr)))
        self.device = int(device)
        self._dbs: list[Database] = []
        self._asm: list["Assembly"] = []

    def set_option(self, key: str, value: int) -> None:
        check(lib().sw_set_option(self.ptr, key.encode(), int(value)), self.ptr)

    def load_db(self, codes, offsets, alphabet_size: int = 24, stream=None, out_index=None,
                out_n: int | None = None) -> Database:
        """sw_load_db, or sw_load_db_mapped when out_index is given: the scores of
        sequence d then land in column out_index[d] of rows of out_n columns."""
        codes = _host(codes, np.uint8)
        offsets = _host(offsets, np.int64)
        n = len(offsets) - 1
        out = ctypes.c_void_p()
        if out_index is None:
            check(lib().sw_load_db(self.ptr, _vp(codes) if codes.size else None, _vp(offsets), n, int(alphabet_size),
                                   _stream_ptr(stream), ctypes.byref(out)), self.ptr)
        else:
            oi = _host(out_index, np.int64)
            check(lib().sw_load_db_mapped(self.ptr, _vp(codes) if codes.size else None, _vp(offsets), n,
                                          int(alphabet_size), _vp(oi) if oi.size else None, int(out_n),
                                          _stream_ptr(stream), ctypes.byref(out)), self.ptr)
        db = Database(self, out, n)
        db.out_n = n if out_index is None else int(out_n)
        db.mapped = out_index is not None
        db.seq_lens = np.diff(offsets)
        self._dbs.append(db)
        return db

    def search(self, q_codes, q_offsets, db: Database, matrix, gap_open: int = 10, gap_extend: int = 2,
               out=None, stream=None):
        """int32 scores[Q][N] in the caller's DB order.

        out: None -> a new torch.int32 CUDA tensor (stream-ordered) if torch has CUDA, else a numpy array;
             a torch CUDA tensor -> written in place on `stream` (caller synchronizes);
             a numpy array -> host output, returned after the copy completes.
        """
        q_codes = _host(q_codes, np.uint8)
        q_offsets = _host(q_offsets, np.int64)
        matrix = _host(matrix, np.int8)
        nq = len(q_offsets) - 1
        N = getattr(db, "out_n", db.n_seqs)
        if out is None:
            if torch is not None and torch.cuda.is_available():
                # a mapped DB writes only its own columns: the rest must not be garbage
                alloc = torch.zeros if getattr(db, "mapped", False) else torch.empty
                out = alloc((nq, N), dtype=torch.int32, device=f"cuda:{self.device}")
            else:
                out = np.zeros((nq, N), dtype=np.int32)
        if torch is not None and isinstance(out, torch.Tensor):
            if out.dtype != torch.int32 or not out.is_contiguous() or tuple(out.shape) != (nq, N):
                raise ValueError(f"search: out must be a contiguous int32 tensor of shape {(nq, N)}")
            if out.is_cuda and out.device.index != self.device:
                raise ValueError(f"search: out is on cuda:{out.device.index}, the handle on cuda:{self.device}")
            if not out.is_cuda and not out.is_pinned():
                out_np = out.numpy()                     # host tensor: written through its numpy view
                optr = _vp(out_np)
            else:
                optr = ctypes.c_void_p(out.data_ptr())
        else:
            if not isinstance(out, np.ndarray) or out.dtype != np.int32 or not out.flags.c_contiguous \
                    or out.shape != (nq, N) or not out.flags.writeable:
                raise ValueError(f"search: out must be a writeable C-contiguous int32 array of shape {(nq, N)}")
            optr = _vp(out)
        check(lib().sw_search(self.ptr, _vp(q_codes) if q_codes.size else None, _vp(q_offsets), nq, db.ptr,
                              _vp(matrix), int(gap_open), int(gap_extend), optr, _stream_ptr(stream)), self.ptr)
        return out

    def align(self, q_codes, q_offsets, db: Database, pairs, matrix, gap_open: int = 10, gap_extend: int = 2,
              stream=None):
        """sw_align: best local alignment of each (query index, DB index) pair.

        Returns a list of (score, q_begin, q_end, d_begin, d_end, ops), ops the
        run-length operations (len << 2 | op; op 0 = M, 1 = I, 2 = D), start to end.
        """
        q_codes = _host(q_codes, np.uint8)
        q_offsets = _host(q_offsets, np.int64)
        matrix = _host(matrix, np.int8)
        pairs = _host(pairs, np.int32).reshape(-1, 2)
        nq = len(q_offsets) - 1
        n = len(pairs)
        if n == 0:
            return []
        info_lens = self._seq_lens(db)
        qlens = np.diff(q_offsets)
        caps = qlens[pairs[:, 0].clip(0, max(nq - 1, 0))] + info_lens[pairs[:, 1].clip(0, len(info_lens) - 1)]
        offs = np.zeros(n + 1, dtype=np.int64)
        np.cumsum(caps, out=offs[1:])
        ops = np.zeros(max(int(offs[-1]), 1), dtype=np.uint32)
        out5 = np.zeros((n, 5), dtype=np.int32)
        nops = np.zeros(n, dtype=np.int32)
        check(lib().sw_align(self.ptr, _vp(q_codes) if q_codes.size else None, _vp(q_offsets), nq, db.ptr,
                             _vp(pairs), n, _vp(matrix), int(gap_open), int(gap_extend), _vp(out5), _vp(ops),
                             _vp(offs), _vp(nops), _stream_ptr(stream)), self.ptr)
        return [tuple(int(x) for x in out5[k]) + ([int(x) for x in ops[offs[k]:offs[k] + nops[k]]],)
                for k in range(n)]

    def _seq_lens(self, db: Database) -> np.ndarray:
        lens = getattr(db, "seq_lens", None)
        if lens is None:
            raise ValueError("align: load the DB through Handle.load_db (sequence lengths needed)")
        return lens

    def assembly(self, blocks, rows, cols, n_queries: int, n_cols: int) -> "Assembly":
        """sw_assembly_create: blocks = int64[n][5] (src_off, row_off, col_off, n_rows, n_cols),
        rows = int32 query indices, cols = int64 DB columns (caller order)."""
        b = _host(blocks, np.int64).reshape(-1, 5)
        rows = _host(rows, np.int32)
        cols = _host(cols, np.int64)
        tab = (Block * max(len(b), 1))()
        for i, x in enumerate(b):
            tab[i] = Block(*[int(v) for v in x])
        out = ctypes.c_void_p()
        check(lib().sw_assembly_create(self.ptr, ctypes.cast(tab, ctypes.c_void_p), len(b),
                                       _vp(rows) if rows.size else None, len(rows),
                                       _vp(cols) if cols.size else None, len(cols), int(n_queries), int(n_cols),
                                       ctypes.byref(out)), self.ptr)
        a = Assembly(self, out)
        self._asm.append(a)
        return a

    def last_stats(self) -> dict:
        s = Stats()
        check(lib().sw_last_stats(self.ptr, ctypes.byref(s)), self.ptr)
        return {f: getattr(s, f) for f, _ in Stats._fields_}

    def close(self) -> None:
        if self.ptr:
            lib().sw_free(self.ptr)
            self.ptr = None
            for d in self._dbs:
                d.ptr = None
            for a in self._asm:
                a.ptr = None

    def __enter__(self):
        return self

    def __exit__(self, *exc):
        self.close()

    def __del__(self):
        try:
            self.close()
        except Exception:
            pass


def encode_ascii(s: str) -> np.ndarray:
    """sw_encode_ascii: protein string -> NCBI codes (unknown -> X)."""
    b = s.encode("ascii", "replace")
    out = np.zeros(len(b), dtype=np.uint8)
    check(lib().sw_encode_ascii(b, len(b), _vp(out) if len(b) else None))
    return out


def search_cpu(q_codes, q_offsets, db_codes, db_offsets, matrix, gap_open: int = 10, gap_extend: int = 2,
               alphabet_size: int = 24, n_threads: int = 1) -> np.ndarray:
    """sw_search_cpu: a CPU-type PE of the hybrid SWDUAL (host AVX2 kernel), int32[Q, N].

    A scheduling target for tasks the dual approximation places on CPUs, not a
    fallback of Handle.search (which never routes here)."""
    q_codes = _host(q_codes, np.uint8)
    q_offsets = _host(q_offsets, np.int64)
    db_codes = _host(db_codes, np.uint8)
    db_offsets = _host(db_offsets, np.int64)
    matrix = _host(matrix, np.int8)
    nq, n = len(q_offsets) - 1, len(db_offsets) - 1
    out = np.zeros((nq, n), dtype=np.int32)
    check(lib().sw_search_cpu(_vp(q_codes) if q_codes.size else None, _vp(q_offsets), nq,
                              _vp(db_codes) if db_codes.size else None, _vp(db_offsets), n, int(alphabet_size),
                              _vp(matrix), int(gap_open), int(gap_extend), int(n_threads), _vp(out) if out.size else None))
    return out


def encode_nucleotide(s: str) -> np.ndarray:
    """sw_encode_nucleotide: DNA/RNA string -> codes A 0, C 1, G 2, T/U 3, other 4."""
    b = s.encode("ascii", "replace")
    out = np.zeros(len(b), dtype=np.uint8)
    check(lib().sw_encode_nucleotide(b, len(b), _vp(out) if len(b) else None))
    return out


def schedule_dual(p_cpu, p_gpu, n_cpu: int, n_gpu: int, variant: str = "greedy"):
    """sw_schedule_dual (variant "greedy": the 2-approximation) or sw_schedule_dual_dp
    (variant "dp": the DP-knapsack refinement): (pe int32[n], makespan, lambda);
    PEs 0..n_cpu-1 are CPUs, then GPUs."""
    pc = _host(p_cpu, np.float64)
    pg = _host(p_gpu, np.float64)
    n = len(pc)
    pe = np.full(n, -1, dtype=np.int32)
    mk, lam = ctypes.c_double(), ctypes.c_double()
    fn = {"greedy": lib().sw_schedule_dual, "dp": lib().sw_schedule_dual_dp}[variant]
    check(fn(n, _vp(pc) if n else None, _vp(pg) if n else None, int(n_cpu), int(n_gpu),
                                 _vp(pe) if n else None, ctypes.byref(mk), ctypes.byref(lam)))
    return pe, mk.value, lam.value
