"""Seeded synthetic inputs shared by the oracle tests, the GPU tests and bench.py.

This module holds NONE of the method's arithmetic (no sampling, no
orthogonalisation, no pivoting): it only builds test matrices A = U Sigma V^T
with known singular values, shaped like the paper's workloads (Sec. 6,
Table 1).  See DESIGN.md §5 for the recipe.
"""

from .matrices import (  # noqa: F401
    LAWS, singular_values, haar_orthogonal, make_matrix, make_matrix_torch, matrix_spec,
)
