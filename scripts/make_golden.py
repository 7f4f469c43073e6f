"""Write the oracle-derived regression fixtures under tests/golden/ (calls only oracle/)."""
import os
import sys

import numpy as np

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
from oracle import philox  # noqa: E402

om = philox.omega(4, 0, 16, 0x5C15)
np.savetxt(os.path.join(ROOT, "tests", "golden", "omega_seed5C15_4x16.txt"), om, fmt="%.17g",
           header="oracle.philox.omega(4, 0, 16, seed=0x5C15): RS-BM32 binary32 normals widened to binary64")
