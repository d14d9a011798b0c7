"""CPU-only tests of the product library's host side: the C ABI loads and exports
every symbol include/swdual.h declares, the host packer, the ASCII encoder, the
BLOSUM62 tables, and sw_init failing cleanly without a GPU."""
import ctypes
import os
import re

import numpy as np
import pytest

import paper_conf_icpp_kedad_sidhoummmmt14_b200 as sw
from paper_conf_icpp_kedad_sidhoummmmt14_b200 import _lib
from oracle.blosum62 import blosum62 as oracle_b62, ALPHABET as ORACLE_ALPHABET

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


def _header_symbols():
    txt = open(os.path.join(ROOT, "include", "swdual.h")).read()
    txt = re.sub(r"/\*.*?\*/", "", txt, flags=re.S)
    return sorted(set(re.findall(r"\b(sw_[a-z_0-9]+)\s*\(", txt)))


def test_library_exports_every_header_symbol():
    L = _lib.lib()
    syms = _header_symbols()
    assert "sw_search" in syms and "sw_load_db" in syms
    for s in syms:
        assert hasattr(L, s), s
    assert set(_lib.EXPORTS) <= set(syms)


def test_init_without_gpu_fails_cleanly():
    import torch
    if torch.cuda.is_available():
        pytest.skip("GPU present")
    with pytest.raises(sw.SWError) as e:
        sw.Handle(0)
    assert e.value.code in (_lib.SW_ECUDA, _lib.SW_EINVAL)


class SwPair(ctypes.Structure):
    _fields_ = [("off", ctypes.c_int64), ("len", ctypes.c_int32), ("id0", ctypes.c_int32),
                ("id1", ctypes.c_int32), ("pad_", ctypes.c_int32)]


def pack(codes, off, alpha=24, t_long=3000):
    L = _lib.lib()
    L.sw_pack_db_host.restype = ctypes.c_int32
    V = ctypes.c_void_p
    L.sw_pack_db_host.argtypes = [V, V, ctypes.c_int64, ctypes.c_int32, ctypes.c_int64, V,
                                  ctypes.POINTER(ctypes.c_int64), V, ctypes.POINTER(ctypes.c_int64),
                                  ctypes.POINTER(ctypes.c_int64)]
    codes = np.ascontiguousarray(codes, np.uint8)
    off = np.ascontiguousarray(off, np.int64)
    npairs, nw, nl = ctypes.c_int64(), ctypes.c_int64(), ctypes.c_int64()
    cp = codes.ctypes.data_as(V) if codes.size else None
    rc = L.sw_pack_db_host(cp, off.ctypes.data_as(V), len(off) - 1, alpha, t_long, None,
                           ctypes.byref(npairs), None, ctypes.byref(nw), ctypes.byref(nl))
    if rc != 0:
        return rc, None, None, None
    pairs = (SwPair * max(1, npairs.value))()
    stream = np.zeros(nw.value, np.uint16)
    rc = L.sw_pack_db_host(cp, off.ctypes.data_as(V), len(off) - 1, alpha, t_long, ctypes.cast(pairs, V),
                           ctypes.byref(npairs), stream.ctypes.data_as(V), ctypes.byref(nw), ctypes.byref(nl))
    return rc, list(pairs)[:npairs.value], stream, nl.value


def _rand_db(rng, n, lmax, alpha=24, zero_frac=0.05):
    lens = rng.integers(1, lmax, size=n)
    lens[rng.random(n) < zero_frac] = 0
    off = np.zeros(n + 1, np.int64)
    np.cumsum(lens, out=off[1:])
    return rng.integers(0, alpha, size=int(off[-1])).astype(np.uint8), off


@pytest.mark.parametrize("seed", range(3))
def test_packer_roundtrip_and_order(seed):
    rng = np.random.default_rng(seed)
    codes, off = _rand_db(rng, 501, 900)
    rc, pairs, stream, n_long = pack(codes, off, t_long=600)
    assert rc == 0
    lens = np.diff(off)
    nonempty = np.flatnonzero(lens > 0)
    ids = [p.id0 for p in pairs] + [p.id1 for p in pairs if p.id1 >= 0]
    # every non-empty sequence exactly once (a permutation), empties absent
    assert sorted(ids) == sorted(nonempty.tolist())
    seq_order = []
    for p in pairs:
        seq_order += [p.id0] + ([p.id1] if p.id1 >= 0 else [])
    sl = lens[seq_order]
    assert np.all(np.diff(sl) <= 0)                                # longest first
    for a, b in zip(seq_order, seq_order[1:]):                     # ties by caller index
        if lens[a] == lens[b]:
            assert a < b
    pad = 24
    prev_end = 0
    for k, p in enumerate(pairs):
        assert p.off == prev_end and p.len % 4 == 0 and p.off % 4 == 0
        prev_end = p.off + p.len
        w = stream[p.off:p.off + p.len]
        lo, hi = (w & 0xFF).astype(np.uint8), (w >> 8).astype(np.uint8)
        l0 = lens[p.id0]
        assert p.len == (l0 + 3) // 4 * 4
        np.testing.assert_array_equal(lo[:l0], codes[off[p.id0]:off[p.id0 + 1]])
        assert np.all(lo[l0:] == pad)
        if p.id1 >= 0:
            l1 = lens[p.id1]
            np.testing.assert_array_equal(hi[:l1], codes[off[p.id1]:off[p.id1 + 1]])
            assert np.all(hi[l1:] == pad)
        else:
            assert np.all(hi == pad)
        assert (k < n_long) == (l0 > 600)
    # padding overhead stays small after the sort
    assert 2 * prev_end <= 1.02 * lens.sum() + 8 * len(pairs)


def test_packer_edges_and_errors():
    rc, pairs, stream, nl = pack(np.zeros(0, np.uint8), np.array([0, 0, 0], np.int64))
    assert rc == 0 and pairs == []
    rc, *_ = pack(np.array([3, 24], np.uint8), np.array([0, 2], np.int64))
    assert rc == _lib.SW_EINVAL                      # code >= alphabet
    rc, *_ = pack(np.array([3, 2], np.uint8), np.array([0, 2, 1], np.int64))
    assert rc == _lib.SW_EINVAL                      # decreasing offsets
    rc, *_ = pack(np.array([3, 2], np.uint8), np.array([0, 2], np.int64), alpha=33)
    assert rc == _lib.SW_EINVAL
    # offsets need not start at 0
    codes = np.arange(10, dtype=np.uint8) % 20
    rc, pairs, stream, _ = pack(codes, np.array([3, 5, 10], np.int64))
    assert rc == 0 and len(pairs) == 1 and pairs[0].id0 == 1 and pairs[0].id1 == 0


def test_encode_ascii():
    got = sw.encode_ascii("ARNDCQEGHILKMFPSTWYVBZX*arndUuOoJ?")
    exp = list(range(24)) + [0, 1, 2, 3, 4, 4, 11, 11, 22, 22]
    assert got.tolist() == exp


def test_encode_nucleotide_and_matrix():
    got = sw.encode_nucleotide("ACGTUacgtuNnRY-")
    assert got.tolist() == [0, 1, 2, 3, 3, 0, 1, 2, 3, 3, 4, 4, 4, 4, 4]
    M = sw.nucleotide_matrix(1, -1)
    assert M.shape == (5, 5) and M.dtype == np.int8
    assert all(M[a, a] == 1 for a in range(4)) and M[4, 4] == -1
    assert (M[~np.eye(5, dtype=bool)] == -1).all()


def test_blosum62_tables():
    """The product's (lower-triangle) and the oracle's (full) transcriptions agree,
    and the table has BLOSUM62's known structure."""
    P = sw.blosum62().astype(np.int32)
    O = oracle_b62()
    assert sw.ALPHABET == ORACLE_ALPHABET == "ARNDCQEGHILKMFPSTWYVBZX*"
    np.testing.assert_array_equal(P, O)
    assert np.array_equal(O, O.T)
    assert np.diag(O).tolist() == [4, 5, 6, 6, 9, 5, 5, 6, 8, 4, 4, 5, 5, 6, 7, 4, 5, 11, 7, 4, 4, 4, -1, 1]
    assert O.min() == -4 and O.max() == 11
    std = O[:20, :20]
    assert all(std[i].argmax() == i for i in range(20))
