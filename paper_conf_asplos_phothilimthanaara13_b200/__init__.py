"""B200-native SeparableConvolution (Phothilimthana et al., ASPLOS'13, Fig. 1).

The compute path is ``libsepconv.so`` (hand-written sm_100a CUDA behind a C ABI,
``include/sepconv.h``); :mod:`.sepconv` is a thin ctypes binding with the same
names.  :mod:`.synth` draws seeded synthetic inputs.
"""
__all__ = ["sepconv", "synth"]
