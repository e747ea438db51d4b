"""B200-native GPMA+ (Sha et al., PVLDB 2017): a C-ABI sm_100a library + thin binding.

The compute lives in ``csrc/*.cu`` compiled to ``lib/libgpma.so`` (see ``build.py``);
``gpma.py`` marshals arguments to the C entry points declared in ``include/gpma.h``.
"""
from .gpma import (  # noqa: F401
    DELETE, DELETE_LAZY, DELETE_REBALANCE, EXPORTS, INSERT, Gpma, GpmaError, lib,
)
from .buildlib import LIB, build  # noqa: F401
