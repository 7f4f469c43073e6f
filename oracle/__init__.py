"""CPU ORACLE for the random-sampling rank-k approximation of Mary et al., SC15.

TEST INFRASTRUCTURE ONLY.  Only ``tests/``, ``__graft_entry__.smoke()`` and
``bench.py`` (its ``cpu_baseline`` leg and ``--impl reference`` arm) may import
anything under ``oracle/``.  The product path (``paper_conf_sc_maryykltd15_b200``)
never imports it and fails loudly when its CUDA library is missing.

The oracle shares no code with the CUDA path: no kernels, headers, helpers,
constant tables or pre/post-processing.  The only module both sides use is
``synth`` (seeded synthetic input matrices), which holds none of the method's
arithmetic.

Citations ``P:L<a>-<b>`` refer to lines of the paper text (PAPER.md, the HAL
extraction of the SC15 paper), with the section / figure / equation named.

Modules
-------
``gemm``     the oracle's own fixed-order matrix product (plain C loop nest in
             ``csrc/gemm.c``, every output summed in increasing k; SURVEY
             §8(c) c-1 step 2) -- every product of the oracle goes through it.
``philox``   Philox4x32-10 and the RS-BM32 Gaussian transform,
             i.e. the PRNG(l, m) of Fig. 2(b) line 2.
``linalg``   Householder QR (sign-normalised), truncated QRCP with recomputed
             norms, back substitution -- the paper's building blocks (§2, §4).
``pipeline`` Fig. 2(a)/(b) step by step: sample, power iteration, QRCP of B,
             T, QR of A P_{1:k}, R, and the error metric of Fig. 6.

Every public function is pinned by ``tests/test_oracle_*.py`` against values
the paper prints, closed forms, brute force or an independent library routine
(LAPACK via numpy/scipy, used in tests only).  See DESIGN.md §4 for the list.
"""

from . import gemm, philox, linalg, pipeline  # noqa: F401
