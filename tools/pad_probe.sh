#!/bin/bash
for L in variants/liblmosem_prev.so ""; do for p in 0 1 2 4 8 16 32 64; do LMOSEM_LIB=$L python tools/pad_probe.py C5 $p 2>&1 | tail -1; done; done
