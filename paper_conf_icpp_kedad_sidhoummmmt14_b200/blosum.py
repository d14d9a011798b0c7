"""Scoring data for the product path: the NCBI protein alphabet and BLOSUM62.

The paper leaves S_ij unnamed; BASELINE.json fixes BLOSUM62
with gap open 10 / extend 2.  The table below is the lower triangle of the NCBI
BLOSUM62 matrix (row letter first), mirrored on load; tests check it against
the oracle's separately transcribed full table.
"""
from __future__ import annotations

import numpy as np

ALPHABET = "ARNDCQEGHILKMFPSTWYVBZX*"
GAP_OPEN, GAP_EXTEND = 10, 2

_LOWER = """
A 4
R -1 5
N -2 0 6
D -2 -2 1 6
C 0 -3 -3 -3 9
Q -1 1 0 0 -3 5
E -1 0 0 2 -4 2 5
G 0 -2 0 -1 -3 -2 -2 6
H -2 0 1 -1 -3 0 0 -2 8
I -1 -3 -3 -3 -1 -3 -3 -4 -3 4
L -1 -2 -3 -4 -1 -2 -3 -4 -3 2 4
K -1 2 0 -1 -3 1 1 -2 -1 -3 -2 5
M -1 -1 -2 -3 -1 0 -2 -3 -2 1 2 -1 5
F -2 -3 -3 -3 -2 -3 -3 -3 -1 0 0 -3 0 6
P -1 -2 -2 -1 -3 -1 -1 -2 -2 -3 -3 -1 -2 -4 7
S 1 -1 1 0 -1 0 0 0 -1 -2 -2 0 -1 -2 -1 4
T 0 -1 0 -1 -1 -1 -1 -2 -2 -1 -1 -1 -1 -2 -1 1 5
W -3 -3 -4 -4 -2 -2 -3 -2 -2 -3 -2 -3 -1 1 -4 -3 -2 11
Y -2 -2 -2 -3 -2 -1 -2 -3 2 -1 -1 -2 -1 3 -3 -2 -2 2 7
V 0 -3 -3 -3 -1 -2 -2 -3 -3 3 1 -2 1 -1 -2 -2 0 -3 -1 4
B -2 -1 3 4 -3 0 1 -1 0 -3 -4 0 -3 -3 -2 0 -1 -4 -3 -3 4
Z -1 0 0 1 -3 3 4 -2 0 -3 -3 1 -1 -3 -1 0 -1 -3 -2 -2 1 4
X 0 -1 -1 -1 -2 -1 -1 -1 -1 -1 -1 -1 -1 -1 -2 0 0 -2 -1 -1 -1 -1 -1
* -4 -4 -4 -4 -4 -4 -4 -4 -4 -4 -4 -4 -4 -4 -4 -4 -4 -4 -4 -4 -4 -4 -4 1
"""


def blosum62() -> np.ndarray:
    """24 x 24 int8 BLOSUM62 in ALPHABET order (row = query letter)."""
    M = np.zeros((24, 24), dtype=np.int8)
    for i, line in enumerate(_LOWER.strip().splitlines()):
        parts = line.split()
        assert parts[0] == ALPHABET[i]
        vals = [int(v) for v in parts[1:]]
        assert len(vals) == i + 1
        for j, v in enumerate(vals):
            M[i, j] = M[j, i] = v
    return M


NUCLEOTIDES = "ACGTN"  # sw_encode_nucleotide codes 0..4 (U shares T's code)


def nucleotide_matrix(match: int = 1, mismatch: int = -1, n_score: int = None) -> np.ndarray:
    """5 x 5 int8 match/mismatch matrix over ACGTN (ma for
    identical bases, mi otherwise; Fig. 1 uses ma = +1, mi = -1).  N scores
    n_score against everything (default: mismatch)."""
    M = np.full((5, 5), mismatch, dtype=np.int8)
    np.fill_diagonal(M, match)
    M[4, :] = M[:, 4] = mismatch if n_score is None else n_score
    return M
