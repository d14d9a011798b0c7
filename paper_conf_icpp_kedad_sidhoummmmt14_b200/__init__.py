"""B200-native SWDUAL hot path: many-query x database Smith-Waterman/Gotoh
scoring (Kedad-Sidhoum et al., ICPP 2014) as a C-ABI CUDA library for sm_100a.

The library is libswdual.so (include/swdual.h); this package is its thin
binding (api.py), the BLOSUM62 table (blosum.py) and the multi-GPU shard +
gather layer (dist.py).
"""
from .api import Database, Handle, encode_ascii, encode_nucleotide, schedule_dual, search_cpu
from ._lib import SWError, LIB_PATH
from .blosum import ALPHABET, GAP_EXTEND, GAP_OPEN, NUCLEOTIDES, blosum62, nucleotide_matrix

__all__ = ["Database", "Handle", "encode_ascii", "encode_nucleotide", "schedule_dual", "search_cpu", "SWError", "LIB_PATH",
           "ALPHABET", "GAP_OPEN", "GAP_EXTEND", "NUCLEOTIDES", "blosum62", "nucleotide_matrix"]
