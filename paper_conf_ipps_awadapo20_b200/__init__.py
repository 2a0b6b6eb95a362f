"""B200-native dynamic graphs: one hash table per vertex (Awad et al., IPDPS 2020).

The product is the C-ABI library ``libdg.so`` (include/dg.h); this package is its thin
Python binding.  Importing it fails loudly if the library has not been built.
"""
from ._lib import (DG_ERR_BAD_STATE, DG_ERR_CUDA, DG_ERR_INVALID_ARGUMENT, DG_ERR_NCCL,  # noqa: F401
                   DG_ERR_OUT_OF_MEMORY, DG_ERR_UNSUPPORTED, DG_ERR_VERTEX_OUT_OF_RANGE, DG_OK,
                   LIB_PATH, DGError)
from .graph import Graph, RankGroup, get_unique_id  # noqa: F401

__all__ = ["Graph", "RankGroup", "DGError", "get_unique_id", "LIB_PATH"]
