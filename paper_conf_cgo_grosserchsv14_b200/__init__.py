"""B200-native hybrid hexagonal/classical tiled stencils (Grosser et al., CGO'14).

The hot path (dependence analysis, tile validation, launch table, sm_100a phase kernels)
lives in lib/libhexstencil.so behind include/stencil.h; this package is the thin Python
binding (argument marshalling; PyTorch for device memory, streams and process groups)."""
from ._lib import KINDS, StencilError, lib
from .api import Plan, Stencil, run

__all__ = ["KINDS", "Plan", "Stencil", "StencilError", "lib", "run"]
