"""B200-native tiled FP64 Cholesky (Agullo et al., HCW 2015) -- Python binding of the
C-ABI library libchol_b200.so.  See include/chol.h and DESIGN.md."""
from .chol import *  # noqa: F401,F403
from .chol import Plan, CholError, EXPORTED, LIB_PATH  # noqa: F401
