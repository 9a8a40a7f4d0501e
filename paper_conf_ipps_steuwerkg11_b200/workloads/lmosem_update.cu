// LM OSEM image update, the body of Listing 3's second inner loop
// as the customizing function of a Zip (Listing 4):
//   f[j] = c[j] > 0 ? f[j] * c[j] : f[j]
float lmosem_update(float f, float c) { return c > 0.0f ? f * c : f; }
