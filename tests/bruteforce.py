"""Pure-Python brute-force tiler enumeration (independent second check of the oracle).

Enumerates every (repetition r, pattern i) pair with itertools.product and
computes each array coordinate as Python's floor-modulus of
origin + P.r + F.i (Section IV).  Deliberately written
with different machinery than the C oracle (itertools + Python ints + tuple
indexing into numpy), and only usable on tiny arrays.
"""
from __future__ import annotations

import itertools

import numpy as np


def enumerate_pairs(array_shape, rep_shape, pattern_shape, origin, paving, fitting):
    """Yield (r, i, coord) in row-major (r, i) order (Fig. 6 loop order)."""
    ra = len(array_shape)
    for r in itertools.product(*[range(s) for s in rep_shape]):
        for i in itertools.product(*[range(s) for s in pattern_shape]):
            coord = tuple(
                (origin[a]
                 + sum(paving[a][j] * r[j] for j in range(len(rep_shape)))
                 + sum(fitting[a][k] * i[k] for k in range(len(pattern_shape)))) % array_shape[a]
                for a in range(ra))
            yield r, i, coord


def gather(A, rep_shape, pattern_shape, origin, paving, fitting):
    vals = [A[c] for _, _, c in enumerate_pairs(A.shape, rep_shape, pattern_shape, origin, paving, fitting)]
    return np.array(vals, dtype=A.dtype).reshape(tuple(rep_shape) + tuple(pattern_shape))


def scatter(A, G, rep_shape, pattern_shape, origin, paving, fitting):
    out = A.copy()
    flat = G.reshape(-1)
    for n, (_, _, c) in enumerate(enumerate_pairs(A.shape, rep_shape, pattern_shape, origin, paving, fitting)):
        out[c] = flat[n]
    return out


def read_counts(array_shape, rep_shape, pattern_shape, origin, paving, fitting):
    cnt = np.zeros(array_shape, dtype=np.int64)
    for _, _, c in enumerate_pairs(array_shape, rep_shape, pattern_shape, origin, paving, fitting):
        cnt[c] += 1
    return cnt


def random_descriptor(rng, max_array_rank=3, max_rep_rank=3, max_pattern_rank=2,
                      array_dim=(1, 17), rep_dim=(1, 6), pattern_dim=(1, 6), entries=(-4, 9)):
    """SURVEY 8(d) d3 recipe (sizes trimmed for pure Python): random ranks, shapes,
    P/F entries in [-4, 9], origin in [-2s, 2s] so the mod wraps both ways."""
    ra = int(rng.integers(1, max_array_rank + 1))
    rr = int(rng.integers(0, max_rep_rank + 1))
    rp = int(rng.integers(0, max_pattern_rank + 1))
    arr = [int(rng.integers(array_dim[0], array_dim[1] + 1)) for _ in range(ra)]
    # keep the brute force small in rank 3
    if ra == 3:
        arr = [min(s, 7) for s in arr]
    rep = [int(rng.integers(rep_dim[0], rep_dim[1] + 1)) for _ in range(rr)]
    pat = [int(rng.integers(pattern_dim[0], pattern_dim[1] + 1)) for _ in range(rp)]
    origin = [int(rng.integers(-2 * s, 2 * s + 1)) for s in arr]
    P = [[int(rng.integers(entries[0], entries[1] + 1)) for _ in range(rr)] for _ in range(ra)]
    F = [[int(rng.integers(entries[0], entries[1] + 1)) for _ in range(rp)] for _ in range(ra)]
    return dict(array_shape=arr, rep_shape=rep, pattern_shape=pat, origin=origin, paving=P, fitting=F)
