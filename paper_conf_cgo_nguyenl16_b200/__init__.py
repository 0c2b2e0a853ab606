"""B200-native executor for synchronous-dataflow stream graphs (Nguyen & Lee, CGO'16).

The product is the native library libsg.so (C ABI: include/sg.h).  `sg` is a
thin ctypes binding with the same names (argument marshalling only).
"""
from . import sg  # noqa: F401
