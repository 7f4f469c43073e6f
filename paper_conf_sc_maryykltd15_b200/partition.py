"""1-D block-row partition of A over ranks (reading R12 in DESIGN.md).

Rank r owns the contiguous rows [r0, r1) of the global m x n matrix A; the first (m mod N) ranks
get ceil(m/N) rows.  Omega is keyed by global row index, so the rank-local sample is
Omega(:, r0:r1) A(r0:r1, :) and the partials sum to Omega A for any partition.
"""

from __future__ import annotations


def row_split(m: int, nranks: int, rank: int) -> tuple[int, int]:
    if nranks < 1 or not 0 <= rank < nranks or m < 0:
        raise ValueError("bad partition arguments")
    base, extra = divmod(m, nranks)
    r0 = rank * base + min(rank, extra)
    return r0, r0 + base + (1 if rank < extra else 0)


def all_splits(m: int, nranks: int) -> list[tuple[int, int]]:
    return [row_split(m, nranks, r) for r in range(nranks)]
